# Quick GPU iteration: focused parity tests + the affected benches.
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -k "fkjsel or q9 or fkj" > gpurun_out/pytest_quick.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_quick.log
VD_FKG_AGG=match timeout 900 python -m pytest tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -k "q9" >> gpurun_out/pytest_quick.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_quick.log
for agg in atom match; do VD_FKG_AGG=$agg timeout 300 python bench.py --workload q9 --steps 20 --no-cpu-baseline --no-e2e > gpurun_out/q_bench_q9_${agg}.json 2>> gpurun_out/q_bench.err; done
timeout 900 python scripts/sweep.py fig16 > gpurun_out/sweep_fig16.jsonl 2>> gpurun_out/q_bench.err
VD_FKJS_VARIANT=ldg timeout 900 python scripts/sweep.py fig16 > gpurun_out/sweep_fig16_ldg.jsonl 2>> gpurun_out/q_bench.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_fkg -s 1 -c 1 -o gpurun_out/prof_q9 -f python bench.py --workload q9 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q9.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_fkjs -s 1 -c 1 -o gpurun_out/prof_fkjsel -f python bench.py --workload fkjsel --selectivity 1.0 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_fkjsel.log 2>&1
