# Re-validation of HEAD on a fresh box: smoke, every GPU parity test, the
# default bench line, every workload's bench line, the launch list, and
# full ncu captures of the L2-gather fragments (q9, q19 late).
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,memory.total --format=csv > gpurun_out/nvsmi.txt 2>&1
nproc > gpurun_out/nproc.txt
make -j16 > gpurun_out/make.log 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/smoke.log
timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider --durations=15 > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
timeout 600 python bench.py > gpurun_out/bench_q1.json 2> gpurun_out/bench_q1.err
for w in q6 q19 q9 select q15; do timeout 300 python bench.py --workload $w --no-cpu-baseline --no-e2e > gpurun_out/bench_${w}.json 2>> gpurun_out/bench_misc.err; done
timeout 300 python bench.py --workload selpos --selectivity 0.5 --no-cpu-baseline --no-e2e > gpurun_out/bench_selpos.json 2>> gpurun_out/bench_misc.err
timeout 300 python bench.py --workload fkjsel --selectivity 0.5 --no-cpu-baseline --no-e2e > gpurun_out/bench_fkjsel.json 2>> gpurun_out/bench_misc.err
timeout 300 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/bench_ref.json 2>> gpurun_out/bench_misc.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/launches_q1.csv python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_launch.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_fkg -s 1 -c 1 -o gpurun_out/prof_q9 -f python bench.py --workload q9 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q9.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_pipe_late -s 1 -c 1 -o gpurun_out/prof_q19 -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/ncu_q19.log 2>&1

# The N > 1 bench path on one GPU: two ranks sharing cuda:0, partials exchanged over gloo.
for w in q1 q19; do
  timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29511 bench.py --workload $w --gpus 2 --steps 20 --warmup 3 --dist-backend gloo --no-cpu-baseline --no-e2e > gpurun_out/bench_2rank_$w.json 2> gpurun_out/bench_2rank_$w.err
done
ls -la gpurun_out
