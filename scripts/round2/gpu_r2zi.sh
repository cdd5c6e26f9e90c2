# Round 2 (re-entry 3): HEAD validation -- smoke, full GPU suite, default bench, its launch list, ncu of k_pipe_q1_tma
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,memory.total --format=csv > gpurun_out/r2zi_nvsmi.txt 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2zi_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/r2zi_smoke.log
timeout 3000 python -m pytest tests -m gpu -q -p no:cacheprovider --durations=5 > gpurun_out/r2zi_pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/r2zi_pytest_gpu.log
timeout 600 python bench.py > gpurun_out/r2zi_bench_q1.json 2>> gpurun_out/r2zi_bench.err
timeout 900 python bench.py --impl reference > gpurun_out/r2zi_bench_ref.json 2>> gpurun_out/r2zi_bench.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/r2zi_launches_q1.csv python bench.py --steps 3 --warmup 3 --no-cpu-baseline > gpurun_out/r2zi_ncu_launch.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_pipe_q1_tma -s 3 -c 1 -o gpurun_out/r2zi_prof_q1 -f python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/r2zi_ncu_q1.log 2>&1
