# Round 2 (re-entry 3): C1-style latency of the selection by input size (positions + sum, warm)
set -x
mkdir -p gpurun_out
for r in 15360 65536 262144 1048576 4194304; do
  timeout 300 python bench.py --workload c1 --rows $r --steps 100 --no-cpu-baseline >> gpurun_out/r2zv_c1_sizes.jsonl 2>> gpurun_out/r2zv_bench.err
done
