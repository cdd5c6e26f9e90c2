mkdir -p gpurun_out
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_late -s 1 -c 1 -o gpurun_out/prof_q19 -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q19.log 2>&1
