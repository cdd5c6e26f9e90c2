mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_group.py -m gpu -q -p no:cacheprovider -x > gpurun_out/pytest_grp.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_grp.log
timeout 300 python bench.py --workload q15 --no-cpu-baseline --no-e2e > gpurun_out/bench_q15.json 2>> gpurun_out/bench_misc.err
