# Round 2: 64-byte late loads + evict_last group tables; coop selection v2; parity + benches + L2 split
set -x
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_select_coop.py tests/test_gpu_hash.py tests/test_gpu_group.py tests/test_gpu_ops.py tests/test_gpu_pipeline.py tests/test_gpu_materialize.py -m gpu -q -p no:cacheprovider > gpurun_out/r2g_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2g_pytest.log
for s in 0.0001 0.01 0.1 0.5 1.0; do for m in branch predicated; do
  timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline >> gpurun_out/r2g_selpos.jsonl 2>> gpurun_out/r2g_bench.err
done; done
timeout 300 python bench.py --workload c1 > gpurun_out/r2g_bench_c1.json 2>> gpurun_out/r2g_bench.err
timeout 300 python bench.py --workload q15 --no-cpu-baseline > gpurun_out/r2g_bench_q15.json 2>> gpurun_out/r2g_bench.err
timeout 300 python bench.py --workload q15 --grouping hash --no-cpu-baseline > gpurun_out/r2g_bench_q15h.json 2>> gpurun_out/r2g_bench.err
timeout 300 python bench.py --workload q19 --no-cpu-baseline --no-e2e > gpurun_out/r2g_bench_q19.json 2>> gpurun_out/r2g_bench.err
timeout 300 python bench.py --workload fkjsel --selectivity 0.1 --no-cpu-baseline --no-e2e > gpurun_out/r2g_bench_fkjsel.json 2>> gpurun_out/r2g_bench.err
M=dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sectors_srcunit_tex_op_read.sum,lts__t_sectors_srcunit_tex_op_read_lookup_miss.sum,lts__t_sectors_srcunit_tex_op_red.sum,lts__t_sectors_srcunit_tex_op_red_lookup_miss.sum,gpu__time_duration.sum
timeout 600 ncu --metrics $M --clock-control none -k regex:k_grp_fold_iv -s 2 -c 1 --csv --log-file gpurun_out/r2g_q15.csv python bench.py --workload q15 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2g_q15.log 2>&1
timeout 600 ncu --metrics $M --clock-control none -k regex:k_pipe_late -s 2 -c 1 --csv --log-file gpurun_out/r2g_q19.csv python bench.py --workload q19 --steps 2 --warmup 2 --no-cpu-baseline --no-e2e > gpurun_out/r2g_q19.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_coop -s 2 -c 1 -o gpurun_out/r2g_prof_selpos -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2g_ncu.log 2>&1
