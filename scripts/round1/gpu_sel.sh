# Selection iteration: parity tests, both Fig 1 modes, selective sum, launch lists.
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_ops.py tests/test_gpu_fullsize.py tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -k "select or sel" > gpurun_out/pytest_sel.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_sel.log
for m in branch; do timeout 300 python bench.py --workload selpos --selectivity 0.5 --sel-mode $m --no-cpu-baseline --no-e2e > gpurun_out/bench_selpos_$m.json 2>> gpurun_out/bench_misc.err; done
VD_SELECT_BITS=ldg timeout 300 python bench.py --workload selpos --selectivity 0.5 --no-cpu-baseline --no-e2e > gpurun_out/bench_selpos_ldg.json 2>> gpurun_out/bench_misc.err
timeout 300 python bench.py --workload select --selectivity 0.5 --no-cpu-baseline --no-e2e > gpurun_out/bench_select.json 2>> gpurun_out/bench_misc.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_selpos.csv python bench.py --workload selpos --selectivity 0.5 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_launch.log 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_select.csv python bench.py --workload select --selectivity 0.5 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_launch2.log 2>&1
