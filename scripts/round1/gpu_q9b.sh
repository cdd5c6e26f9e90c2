set -x
mkdir -p gpurun_out
rm -f gpurun_out/bench_q9_*.json
timeout 900 python -m pytest tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -k "q9" > gpurun_out/pytest_q9.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_q9.log
for b in 4 8; do VD_FKP_BATCH=$b timeout 300 python bench.py --workload q9 --no-cpu-baseline --no-e2e --steps 50 > gpurun_out/bench_q9_b$b.json 2>> gpurun_out/bench_q9.err; done
VD_FKP_PF=4 timeout 300 python bench.py --workload q9 --no-cpu-baseline --no-e2e --steps 50 > gpurun_out/bench_q9_b4pf4.json 2>> gpurun_out/bench_q9.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_fkg -s 1 -c 1 -o gpurun_out/prof_q9p -f python bench.py --workload q9 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q9p.log 2>&1
