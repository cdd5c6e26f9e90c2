# Round 2: coop phase 1 releases the stage before the ballots; graph replay test
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_select_coop.py tests/test_gpu_dist.py -m gpu -q -p no:cacheprovider > gpurun_out/r2r_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2r_pytest.log
for s in 0.0001 0.01 0.1 0.5 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2r_selpos.jsonl 2>> gpurun_out/r2r_bench.err
done; done
VD_SELECT_PHASE1=1 timeout 300 python bench.py --workload selpos --selectivity 0.5 --steps 30 --no-cpu-baseline >> gpurun_out/r2r_selpos_phase1.jsonl 2>> gpurun_out/r2r_bench.err
