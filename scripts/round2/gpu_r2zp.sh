# Round 2 (re-entry 3): Q9 -- shared-memory carveout (more L1 for the 1 MB dimension) and ring depth
set -x
mkdir -p gpurun_out
for c in none 70 80 100; do
  if [ $c = none ]; then unset VD_FKG_CARVE; else export VD_FKG_CARVE=$c; fi
  timeout 600 python bench.py --workload q9 --steps 20 --no-cpu-baseline 2>> gpurun_out/r2zp_bench.err | sed "s/^/carve$c /" >> gpurun_out/r2zp_q9.txt
done
unset VD_FKG_CARVE
timeout 600 ncu --metrics gpu__time_duration.sum,l1tex__t_sector_hit_rate.pct,lts__t_sectors.sum,launch__shared_mem_config_size --clock-control none -k regex:k_pipe_fkg -c 2 --csv python bench.py --workload q9 --steps 1 --warmup 1 --no-cpu-baseline > gpurun_out/r2zp_ncu_default.csv 2>&1
VD_FKG_CARVE=70 timeout 600 ncu --metrics gpu__time_duration.sum,l1tex__t_sector_hit_rate.pct,lts__t_sectors.sum,launch__shared_mem_config_size --clock-control none -k regex:k_pipe_fkg -c 2 --csv python bench.py --workload q9 --steps 1 --warmup 1 --no-cpu-baseline > gpurun_out/r2zp_ncu_70.csv 2>&1
