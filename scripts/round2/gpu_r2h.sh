# Round 2: coop selection v3 (lane-owned words, sparse direct path, 4-deep queue), hash interval path
set -x
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_select_coop.py tests/test_gpu_hash.py tests/test_gpu_ops.py tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -k "select or hash or merge or shards or late or generic" > gpurun_out/r2h_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2h_pytest.log
timeout 900 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -p no:cacheprovider -k "selection" > gpurun_out/r2h_pytest_full.log 2>&1; echo "rc=$?" >> gpurun_out/r2h_pytest_full.log
for s in 0.0001 0.001 0.01 0.05 0.1 0.2 0.5 0.8 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2h_selpos.jsonl 2>> gpurun_out/r2h_bench.err
done; done
timeout 300 python bench.py --workload c1 > gpurun_out/r2h_bench_c1.json 2>> gpurun_out/r2h_bench.err
timeout 300 python bench.py --workload q15 --grouping hash --no-cpu-baseline > gpurun_out/r2h_bench_q15h.json 2>> gpurun_out/r2h_bench.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_coop -s 2 -c 1 -o gpurun_out/r2h_prof_selpos -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2h_ncu.log 2>&1
