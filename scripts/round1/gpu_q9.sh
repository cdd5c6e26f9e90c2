set -x
mkdir -p gpurun_out
for st in 4 3 2; do VD_FKG_STAGES=$st timeout 300 python bench.py --workload q9 --no-cpu-baseline --no-e2e --steps 100 > gpurun_out/bench_q9_st$st.json 2>> gpurun_out/bench_misc.err; done
VD_FKG_STAGES=2 timeout 600 ncu --set full --clock-control none -k regex:k_pipe_fkg -s 1 -c 1 -o gpurun_out/prof_q9_st2 -f python bench.py --workload q9 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q9.log 2>&1
