mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -x > gpurun_out/pytest_pipe.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_pipe.log
for s in 0.01 0.1 0.5; do timeout 300 python bench.py --workload fkjsel --selectivity $s --no-cpu-baseline --no-e2e > gpurun_out/bench_fkjs_$s.json 2>> gpurun_out/bench_misc.err; done
timeout 300 python bench.py --workload q19 --no-cpu-baseline --no-e2e > gpurun_out/bench_q19_late.json 2>> gpurun_out/bench_misc.err
