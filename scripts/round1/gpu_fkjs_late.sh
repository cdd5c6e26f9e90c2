mkdir -p gpurun_out
for s in 0.001 0.01 0.05 0.1 0.2; do
  timeout 300 python bench.py --workload fkjsel --selectivity $s --no-cpu-baseline --no-e2e > gpurun_out/bench_fkjs_$s.json 2>> gpurun_out/bench_misc.err
  VD_FKJS_VARIANT=off VD_LATE=force timeout 300 python bench.py --workload fkjsel --selectivity $s --no-cpu-baseline --no-e2e > gpurun_out/bench_fkjl_$s.json 2>> gpurun_out/bench_misc.err
done
