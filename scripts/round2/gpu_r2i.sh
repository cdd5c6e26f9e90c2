# Round 2: selection phase 2 over 4-chunk groups; warp-parallel grid fold; quick benches
set -x
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_select_coop.py tests/test_gpu_ops.py tests/test_gpu_pipeline.py tests/test_gpu_epsilon.py tests/test_gpu_materialize.py -m gpu -q -p no:cacheprovider > gpurun_out/r2i_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2i_pytest.log
for s in 0.0001 0.001 0.01 0.05 0.1 0.2 0.5 0.8 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2i_selpos.jsonl 2>> gpurun_out/r2i_bench.err
done; done
timeout 300 python bench.py --workload c1 > gpurun_out/r2i_bench_c1.json 2>> gpurun_out/r2i_bench.err
timeout 300 python bench.py --workload q6 --no-cpu-baseline --no-e2e > gpurun_out/r2i_bench_q6.json 2>> gpurun_out/r2i_bench.err
timeout 300 python bench.py --no-cpu-baseline --no-e2e > gpurun_out/r2i_bench_q1.json 2>> gpurun_out/r2i_bench.err
timeout 300 python bench.py --workload select --no-cpu-baseline --no-e2e > gpurun_out/r2i_bench_select.json 2>> gpurun_out/r2i_bench.err
