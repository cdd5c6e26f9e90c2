set -x
mkdir -p gpurun_out
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_sel_write" -s 2 -c 1 -o gpurun_out/prof_sw_v4 -f python bench.py --workload selpos --selectivity 0.5 --steps 1 --warmup 2 --no-cpu-baseline --no-e2e > gpurun_out/ncu_sw.log 2>&1
VD_SELECT_WRITE=scalar timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_sel_write" -s 2 -c 1 -o gpurun_out/prof_sw_scalar -f python bench.py --workload selpos --selectivity 0.5 --steps 1 --warmup 2 --no-cpu-baseline --no-e2e >> gpurun_out/ncu_sw.log 2>&1
