# Late-materialisation fragment: parity, Q19 / Q6 / fkjsel bench with and without it, ncu of k_pipe_late.
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -x -k "q19 or star or late or q6 or fkjsel" > gpurun_out/pytest_late.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_late.log
timeout 300 python bench.py --workload q19 --no-cpu-baseline --no-e2e > gpurun_out/bench_q19_late.json 2>> gpurun_out/bench_misc.err
VD_LATE=force timeout 300 python bench.py --workload q6 --no-cpu-baseline --no-e2e > gpurun_out/bench_q6_late.json 2>> gpurun_out/bench_misc.err
VD_FKJS_VARIANT=off timeout 300 python bench.py --workload fkjsel --no-cpu-baseline --no-e2e > gpurun_out/bench_fkjsel_late.json 2>> gpurun_out/bench_misc.err
timeout 300 python bench.py --workload fkjsel --no-cpu-baseline --no-e2e > gpurun_out/bench_fkjsel.json 2>> gpurun_out/bench_misc.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_late -s 1 -c 1 -o gpurun_out/prof_q19_late -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q19.log 2>&1
