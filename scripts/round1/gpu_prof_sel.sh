# Full ncu captures of the selection kernels and the selective-sum fragment.
set -x
mkdir -p gpurun_out
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_sel_bits_vec|k_sel_write" -s 4 -c 2 -o gpurun_out/prof_selpos -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_selpos.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_selsum -s 2 -c 1 -o gpurun_out/prof_select -f python bench.py --workload select --selectivity 0.5 --steps 1 --warmup 2 --no-cpu-baseline --no-e2e > gpurun_out/ncu_select.log 2>&1
