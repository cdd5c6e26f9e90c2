# One GPU check round: smoke, all parity tests, benches, sweeps, ncu launch list + full captures.
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,memory.total --format=csv > gpurun_out/nvsmi.txt 2>&1
nproc > gpurun_out/nproc.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/smoke.log
timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider --durations=15 > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
timeout 600 python bench.py > gpurun_out/bench_q1.json 2> gpurun_out/bench_q1.err
for w in q6 q19 q9; do timeout 300 python bench.py --workload $w --no-cpu-baseline --no-e2e --steps 50 > gpurun_out/bench_${w}.json 2>> gpurun_out/bench_misc.err; done
timeout 900 python scripts/sweep.py fig1 > gpurun_out/sweep_fig1.jsonl 2>> gpurun_out/bench_misc.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/launches_q1.csv python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_launch.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_pipe_q1 -s 2 -c 1 -o gpurun_out/prof_q1 -f python bench.py --steps 2 --warmup 2 --no-cpu-baseline --no-e2e > gpurun_out/ncu_full.log 2>&1
timeout 600 ncu --set full --clock-control none -k regex:k_pipe_scalar -s 1 -c 1 -o gpurun_out/prof_q6 -f python bench.py --workload q6 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q6.log 2>&1
timeout 600 ncu --set full --clock-control none -k regex:k_pipe_fkg -s 1 -c 1 -o gpurun_out/prof_q9 -f python bench.py --workload q9 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q9.log 2>&1
timeout 600 ncu --set full --clock-control none -k regex:k_pipe_gf -s 1 -c 1 -o gpurun_out/prof_q19 -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q19.log 2>&1
timeout 600 ncu --set full --clock-control none -k regex:k_sel_ -s 3 -c 3 -o gpurun_out/prof_selpos -f python bench.py --workload selpos --selectivity 0.5 --steps 1 --warmup 1 > gpurun_out/ncu_selpos.log 2>&1
ls -la gpurun_out
