# Position pass iteration: selection parity, selpos bench at 3 selectivities, launch list.
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -x -k "select" > gpurun_out/pytest_sel.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_sel.log
for s in 0.0001 0.5 1.0; do timeout 300 python bench.py --workload selpos --selectivity $s --no-cpu-baseline --no-e2e > gpurun_out/bench_selpos_$s.json 2>> gpurun_out/bench_misc.err; done
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 40 --csv --log-file gpurun_out/launches_selpos.csv python bench.py --workload selpos --selectivity 0.5 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_launch.log 2>&1
