# Round 2 (re-entry 3): k_sel_lag LAG 16 vs 4, lane-owned threshold 640
set -x
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_select_coop.py -m gpu -q -x -p no:cacheprovider -k "large or lag" > gpurun_out/r2za_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2za_pytest.log
for L in 16 4; do for s in 0.0001 0.01 0.1 0.5 1.0; do for m in branch predicated; do
  VD_SEL_LAG=$L timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2za_bench.err | sed "s/^/lag$L /" >> gpurun_out/r2za_selpos.txt
done; done; done
for s in 0.1 0.5 1.0; do for m in branch predicated; do
  VD_SEL_MID=640 timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2za_bench.err | sed "s/^/lag16-mid640 /" >> gpurun_out/r2za_selpos.txt
done; done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_lag -s 2 -c 1 -o gpurun_out/r2za_prof_lag0001 -f python bench.py --workload selpos --selectivity 0.0001 --steps 2 --warmup 2 --no-cpu-baseline >> gpurun_out/r2za_ncu.log 2>&1
