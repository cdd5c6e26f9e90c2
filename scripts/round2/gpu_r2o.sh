# Round 2: full GPU suite at HEAD, ncu of the Q1 kernel / launch list of the default bench, selection s=0.1 profile, q15 hash
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,memory.total --format=csv > gpurun_out/r2o_nvsmi.txt 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2o_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/r2o_smoke.log
timeout 3000 python -m pytest tests -m gpu -q -p no:cacheprovider --durations=10 > gpurun_out/r2o_pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/r2o_pytest_gpu.log
timeout 300 python bench.py --workload q15 --grouping hash --no-cpu-baseline > gpurun_out/r2o_bench_q15h.json 2>> gpurun_out/r2o_bench.err
timeout 300 python bench.py --workload q15 --no-cpu-baseline > gpurun_out/r2o_bench_q15.json 2>> gpurun_out/r2o_bench.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/r2o_launches_q1.csv python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/r2o_ncu_launch.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_q1_tma -s 2 -c 1 -o gpurun_out/r2o_prof_q1 -f python bench.py --steps 1 --warmup 2 --no-cpu-baseline --no-e2e > gpurun_out/r2o_ncu_q1.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_coop -s 2 -c 1 -o gpurun_out/r2o_prof_selpos01 -f python bench.py --workload selpos --selectivity 0.1 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2o_ncu_sel.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_hg_fold_iv -s 1 -c 1 -o gpurun_out/r2o_prof_q15h -f python bench.py --workload q15 --grouping hash --steps 1 --warmup 1 --no-cpu-baseline > gpurun_out/r2o_ncu_q15h.log 2>&1
