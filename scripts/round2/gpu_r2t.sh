# Round 2: k_sel_stream vs k_sel_coop, same box
set -x
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_select_coop.py -m gpu -q -x -p no:cacheprovider > gpurun_out/r2t_pytest_4.log 2>&1; echo "rc=$?" >> gpurun_out/r2t_pytest_4.log
for c in stream coop; do for s in 0.0001 0.01 0.1 0.5 1.0; do for m in branch predicated; do
  VD_SELECT_KERNEL=$c timeout 300 python bench.py --workload selpos --selectivity $s --sel-mode $m --steps 30 --no-cpu-baseline 2>> gpurun_out/r2t_bench.err | sed "s/^/$c /" >> gpurun_out/r2t_selpos.txt
done; done; done
