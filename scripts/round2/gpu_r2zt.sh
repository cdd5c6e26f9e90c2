# Round 2 (re-entry 3): final HEAD validation after the selection defaults change -- smoke, full GPU suite, default bench, repeat points
set -x
mkdir -p gpurun_out
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2zt_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/r2zt_smoke.log
timeout 3000 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/r2zt_pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/r2zt_pytest_gpu.log
timeout 600 python bench.py > gpurun_out/r2zt_bench_q1.json 2>> gpurun_out/r2zt_bench.err
for i in 1 2 3; do for s in 0.01 0.1; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode predicated --steps 30 --no-cpu-baseline >> gpurun_out/r2zt_selpos_repeat.jsonl 2>> gpurun_out/r2zt_bench.err
done; done
