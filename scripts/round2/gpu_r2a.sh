# Round 2: epsilon / overflow-proof parity, the whole GPU suite, Q1/Q6 bench lines.
set -x
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_epsilon.py -m gpu -q -p no:cacheprovider > gpurun_out/r2a_eps.log 2>&1; echo "rc=$?" >> gpurun_out/r2a_eps.log
timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider -x --durations=10 > gpurun_out/r2a_pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/r2a_pytest_gpu.log
timeout 600 python bench.py --no-cpu-baseline --no-e2e > gpurun_out/r2a_bench_q1.json 2> gpurun_out/r2a_bench.err
timeout 300 python bench.py --workload q6 --no-cpu-baseline --no-e2e > gpurun_out/r2a_bench_q6.json 2>> gpurun_out/r2a_bench.err
