mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -x -k "q9 or fkg" > gpurun_out/pytest_q9.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_q9.log
for st in 2 3 4 6; do VD_FKG_STAGES=$st timeout 300 python bench.py --workload q9 --no-cpu-baseline --no-e2e --steps 200 > gpurun_out/bench_q9_t$st.json 2>> gpurun_out/bench_misc.err; done
