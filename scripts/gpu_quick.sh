# Quick GPU iteration: focused parity tests + the affected benches.
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_ops.py tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -k "select or fkj or selective or fold_select or q6 or q1 or generic or shards or run_alignment" > gpurun_out/pytest_quick.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_quick.log
timeout 300 python bench.py --no-cpu-baseline --no-e2e > gpurun_out/q_bench_q1.json 2> gpurun_out/q_bench.err
timeout 300 python bench.py --workload q6 --no-cpu-baseline --no-e2e > gpurun_out/q_bench_q6.json 2>> gpurun_out/q_bench.err
timeout 300 python bench.py --workload select --no-cpu-baseline --no-e2e > gpurun_out/q_bench_select.json 2>> gpurun_out/q_bench.err
timeout 900 python scripts/sweep.py fig1 > gpurun_out/sweep_fig1.jsonl 2>> gpurun_out/q_bench.err
timeout 900 python scripts/sweep.py fig15 > gpurun_out/sweep_fig15.jsonl 2>> gpurun_out/q_bench.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 40 --csv --log-file gpurun_out/launches_selpos.csv python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 3 > gpurun_out/ncu_launch_selpos.log 2>&1
timeout 600 ncu --set full --clock-control none -k regex:k_sel_ -s 3 -c 3 -o gpurun_out/prof_selpos -f python bench.py --workload selpos --selectivity 0.5 --steps 1 --warmup 1 > gpurun_out/ncu_selpos.log 2>&1
timeout 600 ncu --set full --clock-control none -k regex:k_pipe_selsum -s 1 -c 1 -o gpurun_out/prof_select -f python bench.py --workload select --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_select.log 2>&1
