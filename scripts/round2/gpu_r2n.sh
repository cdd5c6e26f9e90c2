# Round 2: dense branching groups store directly; rounds vs direct threshold sweep
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_select_coop.py tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -k "select" > gpurun_out/r2n_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2n_pytest.log
VD_SELECT_ROUND_MAX=0 timeout 900 python -m pytest tests/test_gpu_select_coop.py -m gpu -q -p no:cacheprovider > gpurun_out/r2n_pytest_direct.log 2>&1; echo "rc=$?" >> gpurun_out/r2n_pytest_direct.log
for rm in 1024 256 0; do for s in 0.01 0.05 0.1 0.2 0.5 1.0; do
  VD_SELECT_ROUND_MAX=$rm timeout 300 python bench.py --workload selpos --selectivity $s --steps 30 --no-cpu-baseline | sed "s/^/$rm /" >> gpurun_out/r2n_selpos.txt 2>> gpurun_out/r2n_bench.err
done; done
