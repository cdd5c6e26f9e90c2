# Session-2 state check: smoke, all GPU parity tests, every bench workload, launch list.
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,memory.total --format=csv > gpurun_out/nvsmi.txt 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/smoke.log
timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider --durations=15 -x > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
timeout 600 python bench.py > gpurun_out/bench_q1.json 2> gpurun_out/bench_q1.err
for w in q6 q19 q9; do timeout 300 python bench.py --workload $w --no-cpu-baseline --no-e2e --steps 50 > gpurun_out/bench_${w}.json 2>> gpurun_out/bench_misc.err; done
for m in branch predicated; do timeout 300 python bench.py --workload selpos --selectivity 0.5 --sel-mode $m --no-cpu-baseline --no-e2e --steps 20 > gpurun_out/bench_selpos_$m.json 2>> gpurun_out/bench_misc.err; done
timeout 300 python bench.py --workload select --selectivity 0.5 --no-cpu-baseline --no-e2e --steps 20 > gpurun_out/bench_select.json 2>> gpurun_out/bench_misc.err
timeout 300 python bench.py --workload fkjsel --selectivity 0.5 --no-cpu-baseline --no-e2e --steps 20 > gpurun_out/bench_fkjsel.json 2>> gpurun_out/bench_misc.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_fkg -s 1 -c 1 -o gpurun_out/prof_q9 -f python bench.py --workload q9 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q9.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_gf -s 1 -c 1 -o gpurun_out/prof_q19 -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q19.log 2>&1
ls -la gpurun_out
