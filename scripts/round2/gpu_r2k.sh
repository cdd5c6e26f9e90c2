# Round 2: the Fig 15 / Fig 16 / Fig 14 sweeps on targets beyond L2, the default bench line, smoke, 2-rank runs
set -x
mkdir -p gpurun_out
for s in 0.0001 0.001 0.01 0.05 0.1 0.2 0.5 0.8 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2k_selpos.jsonl 2>> gpurun_out/r2k_bench.err
done; done
timeout 300 python bench.py --workload c1 > gpurun_out/r2k_bench_c1.json 2>> gpurun_out/r2k_bench.err
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2k_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/r2k_smoke.log
timeout 900 python bench.py > gpurun_out/r2k_bench_q1.json 2> gpurun_out/r2k_bench_q1.err
timeout 300 python bench.py --impl reference --steps 3 --warmup 1 > gpurun_out/r2k_bench_ref.json 2>> gpurun_out/r2k_bench.err
for w in q1 q15; do
  timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29513 bench.py --workload $w --gpus 2 --steps 10 --warmup 3 --dist-backend gloo --no-cpu-baseline --no-e2e > gpurun_out/r2k_bench_2rank_$w.json 2> gpurun_out/r2k_bench_2rank_$w.err
done
timeout 2400 python scripts/sweep.py fig15m > gpurun_out/r2k_sweep_fig15m.jsonl 2>> gpurun_out/r2k_bench.err
timeout 1500 python scripts/sweep.py fig16 > gpurun_out/r2k_sweep_fig16.jsonl 2>> gpurun_out/r2k_bench.err
timeout 900 python scripts/sweep.py fig14 > gpurun_out/r2k_sweep_fig14.jsonl 2>> gpurun_out/r2k_bench.err
