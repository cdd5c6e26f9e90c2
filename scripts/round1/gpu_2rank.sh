# The N > 1 bench path on one GPU: two ranks sharing cuda:0, partials exchanged over gloo.
mkdir -p gpurun_out
for w in q1 q19; do
  timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29511 bench.py --workload $w --gpus 2 --steps 20 --warmup 3 --dist-backend gloo --no-cpu-baseline --no-e2e > gpurun_out/bench_2rank_$w.json 2> gpurun_out/bench_2rank_$w.err
done
