# Round 2 (re-entry 3): selective sum (Fig 15 / C1) with 64 KB tiles x 3 stages vs 32 KB x 6
set -x
mkdir -p gpurun_out
timeout 1500 python -m pytest tests -m gpu -q -x -p no:cacheprovider -k "selsum or select or fig15 or c1 or scalar" > gpurun_out/r2zw_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2zw_pytest.log
for t in 16384 8192 16384 8192; do for s in 0.0001 0.5 1.0; do for m in branch predicated; do
  VD_SELSUM_TILE=$t timeout 300 python bench.py --workload select --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2zw_bench.err | sed "s/^/tile$t /" >> gpurun_out/r2zw_select.txt
done; done; done
