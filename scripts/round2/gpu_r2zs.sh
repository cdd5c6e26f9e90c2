# Round 2 (re-entry 3): k_sel_lag with the branching fixed lane loop by default -- parity + Fig 1 sweep
set -x
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_select_coop.py -m gpu -q -x -p no:cacheprovider > gpurun_out/r2zs_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2zs_pytest.log
for s in 0.0001 0.001 0.01 0.05 0.1 0.2 0.5 0.8 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 2>> gpurun_out/r2zs_bench.err >> gpurun_out/r2zs_selpos.jsonl
done; done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_lag -s 2 -c 1 -o gpurun_out/r2zs_prof_lag05 -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2zs_ncu.log 2>&1
