# One GPU check round: smoke, parity tests, benches, ncu launch list + full capture.
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,memory.total --format=csv > gpurun_out/nvsmi.txt 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/smoke.log
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider --durations=10 > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
timeout 600 python bench.py > gpurun_out/bench_q1.json 2> gpurun_out/bench_q1.err
for w in q6 select; do
  for m in branch predicated; do
    timeout 300 python bench.py --workload $w --sel-mode $m --no-cpu-baseline --no-e2e > gpurun_out/bench_${w}_${m}.json 2>> gpurun_out/bench_misc.err
  done
done
VD_SCALAR_VARIANT=ldg timeout 300 python bench.py --workload q6 --no-cpu-baseline --no-e2e > gpurun_out/bench_q6_ldg.json 2>> gpurun_out/bench_misc.err
for s in 0.01 0.5 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 50 > gpurun_out/bench_selpos_${s}_${m}.json 2>> gpurun_out/bench_misc.err
done; done
for w in q19 q9; do timeout 300 python bench.py --workload $w --steps 20 --no-cpu-baseline --no-e2e > gpurun_out/bench_${w}.json 2>> gpurun_out/bench_misc.err; done
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/launches_q1.csv python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_launch.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_pipe_q1 -s 2 -c 1 -o gpurun_out/prof_q1 -f python bench.py --steps 2 --warmup 2 --no-cpu-baseline --no-e2e > gpurun_out/ncu_full.log 2>&1
timeout 600 ncu --set full --clock-control none -k regex:k_pipe_scalar -s 2 -c 1 -o gpurun_out/prof_q6 -f python bench.py --workload q6 --steps 2 --warmup 2 --no-cpu-baseline --no-e2e > gpurun_out/ncu_full_q6.log 2>&1
ls -la gpurun_out
