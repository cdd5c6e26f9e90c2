mkdir -p gpurun_out
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_write -s 1 -c 1 -o gpurun_out/prof_selw -f python bench.py --workload selpos --selectivity 0.5 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_selw.log 2>&1
