# Round 2: epsilon parity, whole GPU suite, bench lines (q1 with cpu baseline, q6 sf10/sf100, c1, selpos, reference arm)
set -x
mkdir -p gpurun_out
nproc > gpurun_out/nproc.txt; free -g > gpurun_out/free.txt; grep -m1 "model name" /proc/cpuinfo >> gpurun_out/nproc.txt
timeout 600 python -m pytest tests/test_gpu_epsilon.py -m gpu -q -p no:cacheprovider > gpurun_out/r2b_eps.log 2>&1; echo "rc=$?" >> gpurun_out/r2b_eps.log
timeout 3000 python -m pytest tests -m gpu -q -p no:cacheprovider --durations=10 > gpurun_out/r2b_pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/r2b_pytest_gpu.log
timeout 900 python bench.py > gpurun_out/r2b_bench_q1.json 2> gpurun_out/r2b_bench.err
timeout 300 python bench.py --workload q6 --no-e2e > gpurun_out/r2b_bench_q6.json 2>> gpurun_out/r2b_bench.err
timeout 300 python bench.py --workload q6 --sf 100 --no-cpu-baseline > gpurun_out/r2b_bench_q6_sf100.json 2>> gpurun_out/r2b_bench.err
timeout 300 python bench.py --workload c1 > gpurun_out/r2b_bench_c1.json 2>> gpurun_out/r2b_bench.err
timeout 300 python bench.py --workload q19 --no-e2e > gpurun_out/r2b_bench_q19.json 2>> gpurun_out/r2b_bench.err
timeout 300 python bench.py --impl reference --steps 3 --warmup 1 > gpurun_out/r2b_bench_ref.json 2>> gpurun_out/r2b_bench.err
