# Late-materialisation fragment: parity (pipeline tests), Q19 / Q6 bench with and without it, ncu of k_pipe_late.
set -x
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/ -m gpu -q -p no:cacheprovider > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
timeout 300 python bench.py --workload q19 --no-cpu-baseline --no-e2e > gpurun_out/bench_q19_late.json 2>> gpurun_out/bench_misc.err
VD_LATE=off timeout 300 python bench.py --workload q19 --no-cpu-baseline --no-e2e > gpurun_out/bench_q19_star.json 2>> gpurun_out/bench_misc.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_late -s 1 -c 1 -o gpurun_out/prof_q19_late -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q19.log 2>&1
