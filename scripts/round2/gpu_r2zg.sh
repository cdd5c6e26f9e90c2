# Round 2 (re-entry 3): k_sel_lag at every size (C1: 2^20 rows = 69 one-tile CTAs)
set -x
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_select_coop.py tests/test_gpu_ops.py -m gpu -q -x -p no:cacheprovider -k "select or sel" > gpurun_out/r2zg_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2zg_pytest.log
timeout 300 python bench.py --workload c1 --steps 100 --no-cpu-baseline > gpurun_out/r2zg_c1.json 2>> gpurun_out/r2zg_bench.err
for s in 0.0001 0.5; do timeout 300 python bench.py --workload selpos --selectivity $s --steps 30 --no-cpu-baseline >> gpurun_out/r2zg_selpos.jsonl 2>> gpurun_out/r2zg_bench.err; done
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file gpurun_out/r2zg_c1_launches.csv python bench.py --workload c1 --steps 3 --warmup 3 --no-cpu-baseline > gpurun_out/r2zg_c1_ncu.log 2>&1
