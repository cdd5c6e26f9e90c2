# Q19 late fragment quick loop: late parity tests, Q19 bench.
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -x -k "q19 or star or late or fkjsel or q6" > gpurun_out/pytest_late.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_late.log
timeout 300 python bench.py --workload q19 --no-cpu-baseline --no-e2e > gpurun_out/bench_q19_late.json 2>> gpurun_out/bench_misc.err
