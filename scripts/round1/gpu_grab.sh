mkdir -p gpurun_out
for g in 4 8 16 32 64; do VD_LATE_GRAB=$g timeout 300 python bench.py --workload q19 --no-cpu-baseline --no-e2e > gpurun_out/bench_q19_g$g.json 2>> gpurun_out/bench_misc.err; done
