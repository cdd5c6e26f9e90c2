# Round 2 (re-entry 3): k_sel_lag v3 -- producer warp publishes tiles and computes bases (mbarrier handoffs, no CTA barrier per iteration)
set -x
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_select_coop.py -m gpu -q -x -p no:cacheprovider > gpurun_out/r2zb_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2zb_pytest.log
for L in 16 12; do for s in 0.0001 0.01 0.1 0.5 1.0; do for m in branch predicated; do
  VD_SEL_LAG=$L timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2zb_bench.err | sed "s/^/lag$L /" >> gpurun_out/r2zb_selpos.txt
done; done; done
for mid in 640 160; do for s in 0.1 0.5 1.0; do for m in branch predicated; do
  VD_SEL_MID=$mid timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2zb_bench.err | sed "s/^/lag16-mid$mid /" >> gpurun_out/r2zb_selpos.txt
done; done; done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_lag -s 2 -c 1 -o gpurun_out/r2zb_prof_lag05 -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline >> gpurun_out/r2zb_ncu.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_lag -s 2 -c 1 -o gpurun_out/r2zb_prof_lag01 -f python bench.py --workload selpos --selectivity 0.1 --steps 2 --warmup 2 --no-cpu-baseline >> gpurun_out/r2zb_ncu.log 2>&1
