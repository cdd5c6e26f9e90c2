# Round 2: k_sel_stream counting-warp split sweep + ncu of stream (CNT 4, 8) and coop at s=0.5
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_select_coop.py -m gpu -q -x -p no:cacheprovider > gpurun_out/r2w_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2w_pytest.log
for c in 4 6 8; do for s in 0.0001 0.1 0.5 1.0; do for m in branch predicated; do
  VD_SELECT_STREAM_CNT=$c timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2w_bench.err | sed "s/^/cnt$c /" >> gpurun_out/r2w_selpos.txt
done; done; done
for c in 4 8; do
VD_SELECT_STREAM_CNT=$c timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_stream -s 2 -c 1 -o gpurun_out/r2w_prof_stream$c -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2w_ncu_$c.log 2>&1
done
VD_SELECT_KERNEL=coop timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_coop -s 2 -c 1 -o gpurun_out/r2w_prof_coop -f python bench.py --workload selpos --selectivity 0.5 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2w_ncu_coop.log 2>&1
