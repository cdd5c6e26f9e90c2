# Quick GPU iteration: focused parity tests + the affected benches.
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_ops.py tests/test_gpu_pipeline.py tests/test_gpu_dist.py -m gpu -q -p no:cacheprovider -k "select or fkj or selective or fold_select or q6 or q1 or generic or shards or run_alignment or ranks or fold_vs" > gpurun_out/pytest_quick.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_quick.log
timeout 900 python scripts/sweep.py fig1 > gpurun_out/sweep_fig1.jsonl 2>> gpurun_out/q_bench.err
for w in q19 q9; do timeout 300 python bench.py --workload $w --steps 20 --no-cpu-baseline --no-e2e > gpurun_out/q_bench_${w}.json 2>> gpurun_out/q_bench.err; done
timeout 600 ncu --set full --clock-control none -k regex:k_sel_ -s 3 -c 3 -o gpurun_out/prof_selpos -f python bench.py --workload selpos --selectivity 0.5 --steps 1 --warmup 1 > gpurun_out/ncu_selpos.log 2>&1
timeout 600 ncu --set full --clock-control none -k regex:k_pipe_fkg -s 1 -c 1 -o gpurun_out/prof_q9 -f python bench.py --workload q9 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q9.log 2>&1
timeout 600 ncu --set full --clock-control none -k regex:k_pipe_gf -s 1 -c 1 -o gpurun_out/prof_q19 -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q19.log 2>&1
