# Round 2 (re-entry 3): HEAD re-validation -- smoke, full GPU suite, default bench, selection phase-1-only timing
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,memory.total --format=csv > gpurun_out/r2x_nvsmi.txt 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2x_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/r2x_smoke.log
timeout 3000 python -m pytest tests -m gpu -q -p no:cacheprovider --durations=10 > gpurun_out/r2x_pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/r2x_pytest_gpu.log
timeout 600 python bench.py > gpurun_out/r2x_bench_q1.json 2>> gpurun_out/r2x_bench.err
for s in 0.0001 0.1 0.5 1.0; do for m in branch predicated; do
  VD_SELECT_KERNEL=coop VD_SELECT_PHASE1=1 timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2x_bench.err | sed "s/^/coop-p1 /" >> gpurun_out/r2x_selpos.txt
done; done
