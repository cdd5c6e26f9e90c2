# Round 2: fused selection parity + sweeps (fused vs bitmap), device merge, bench lines.
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_select_fused.py tests/test_gpu_merge.py tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -k "select or merge" > gpurun_out/r2c_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2c_pytest.log
timeout 900 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -p no:cacheprovider -k "selection" > gpurun_out/r2c_pytest_full.log 2>&1; echo "rc=$?" >> gpurun_out/r2c_pytest_full.log
timeout 900 python bench.py > gpurun_out/r2c_bench_q1.json 2> gpurun_out/r2c_bench.err
timeout 300 python bench.py --workload c1 > gpurun_out/r2c_bench_c1.json 2>> gpurun_out/r2c_bench.err
timeout 300 python bench.py --workload q6 --no-e2e > gpurun_out/r2c_bench_q6.json 2>> gpurun_out/r2c_bench.err
for s in 0.0001 0.01 0.1 0.5 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2c_selpos_fused.jsonl 2>> gpurun_out/r2c_bench.err
  VD_SELECT_FUSED=0 timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2c_selpos_bitmap.jsonl 2>> gpurun_out/r2c_bench.err
done; done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_fused -s 2 -c 1 -o gpurun_out/r2c_prof_selpos -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2c_ncu.log 2>&1
