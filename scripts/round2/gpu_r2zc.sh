# Round 2 (re-entry 3): k_sel_lag default (LAG 12, predicated lane-owned <= 640): full GPU suite + Fig 1 sweep
set -x
mkdir -p gpurun_out
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2zc_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/r2zc_smoke.log
timeout 3000 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/r2zc_pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/r2zc_pytest_gpu.log
for s in 0.0001 0.001 0.01 0.05 0.1 0.2 0.5 0.8 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 2>> gpurun_out/r2zc_bench.err >> gpurun_out/r2zc_selpos.jsonl
done; done
