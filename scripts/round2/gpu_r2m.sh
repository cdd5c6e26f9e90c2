# Round 2: two-column selective sum on the TMA kernel; selection with 16 decoding warps; Fig 15 sweep again
set -x
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_epsilon.py tests/test_gpu_materialize.py tests/test_gpu_select_coop.py tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider > gpurun_out/r2m_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2m_pytest.log
for s in 0.0001 0.01 0.05 0.1 0.2 0.5 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2m_selpos.jsonl 2>> gpurun_out/r2m_bench.err
done; done
for s in 0.1 0.5; do VD_SELECT_PHASE1=1 timeout 300 python bench.py --workload selpos --selectivity $s --steps 30 --no-cpu-baseline >> gpurun_out/r2m_selpos_phase1.jsonl 2>> gpurun_out/r2m_bench.err; done
timeout 2400 python scripts/sweep.py fig15m > gpurun_out/r2m_sweep_fig15m.jsonl 2>> gpurun_out/r2m_bench.err
