# Round 2: decoupled fused selection, materialising plans, merge; sweeps
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_select_coop.py tests/test_gpu_merge.py tests/test_gpu_materialize.py tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -k "select or merge or materialis or fig15 or q6 or q1 or fk" > gpurun_out/r2d_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2d_pytest.log
timeout 900 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -p no:cacheprovider -k "selection" > gpurun_out/r2d_pytest_full.log 2>&1; echo "rc=$?" >> gpurun_out/r2d_pytest_full.log
for s in 0.0001 0.01 0.1 0.5 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2d_selpos_fused.jsonl 2>> gpurun_out/r2d_bench.err
done; done
timeout 300 python bench.py --workload c1 > gpurun_out/r2d_bench_c1.json 2>> gpurun_out/r2d_bench.err
timeout 900 python bench.py > gpurun_out/r2d_bench_q1.json 2>> gpurun_out/r2d_bench.err
timeout 2400 python scripts/sweep.py fig15m > gpurun_out/r2d_sweep_fig15m.jsonl 2>> gpurun_out/r2d_bench.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_fused -s 2 -c 1 -o gpurun_out/r2d_prof_selpos -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2d_ncu.log 2>&1
