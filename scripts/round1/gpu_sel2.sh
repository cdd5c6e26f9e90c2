set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -k "flag_pass or select_f32" > gpurun_out/pytest_sel.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_sel.log
VD_TILE_ORDER=blocked timeout 900 python -m pytest tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -k "flag_pass or select_f32" >> gpurun_out/pytest_sel.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_sel.log
timeout 300 python bench.py --workload selpos --selectivity 0.5 --no-cpu-baseline --no-e2e > gpurun_out/bench_selpos_strided.json 2>> gpurun_out/bench_misc.err
VD_TILE_ORDER=blocked timeout 300 python bench.py --workload selpos --selectivity 0.5 --no-cpu-baseline --no-e2e > gpurun_out/bench_selpos_blocked.json 2>> gpurun_out/bench_misc.err
VD_TILE_ORDER=blocked timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_selpos_blocked.csv python bench.py --workload selpos --selectivity 0.5 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_launch.log 2>&1
