# Round 2 (re-entry 3): lagged single-pass selection (k_sel_lag) -- parity, sweep vs coop, ncu at s=0.5
set -x
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_select_coop.py -m gpu -q -x -p no:cacheprovider > gpurun_out/r2y_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2y_pytest.log
for c in lag coop; do for s in 0.0001 0.01 0.1 0.5 1.0; do for m in branch predicated; do
  VD_SELECT_KERNEL=$c timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2y_bench.err | sed "s/^/$c /" >> gpurun_out/r2y_selpos.txt
done; done; done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_lag -s 2 -c 1 -o gpurun_out/r2y_prof_lag05 -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2y_ncu.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_lag -s 2 -c 1 -o gpurun_out/r2y_prof_lag001p -f python bench.py --workload selpos --selectivity 0.01 --sel-mode predicated --steps 2 --warmup 2 --no-cpu-baseline >> gpurun_out/r2y_ncu.log 2>&1
for mid in 0 1024; do for s in 0.01 0.1 0.5 1.0; do for m in branch predicated; do
  VD_SEL_MID=$mid timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2y_bench.err | sed "s/^/lag-mid$mid /" >> gpurun_out/r2y_selpos.txt
done; done; done
