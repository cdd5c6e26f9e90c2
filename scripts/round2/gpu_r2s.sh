# Round 2: striped warp-specialised selection (k_sel_stream)
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_select_coop.py tests/test_gpu_ops.py -m gpu -q -x -p no:cacheprovider -k "select" > gpurun_out/r2s_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2s_pytest.log
timeout 600 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -p no:cacheprovider -k "selection" > gpurun_out/r2s_pytest_full.log 2>&1; echo "rc=$?" >> gpurun_out/r2s_pytest_full.log
for s in 0.0001 0.01 0.05 0.1 0.2 0.5 0.8 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2s_selpos.jsonl 2>> gpurun_out/r2s_bench.err
done; done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_stream -s 2 -c 1 -o gpurun_out/r2s_prof_selpos -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2s_ncu.log 2>&1
