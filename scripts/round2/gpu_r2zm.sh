# Round 2 (re-entry 3): late fragment fast round with two rows per thread at 3 CTAs/SM (VD_LATE_PAIR=1) vs one
set -x
mkdir -p gpurun_out
VD_LATE_PAIR=1 timeout 1500 python -m pytest tests/test_gpu_pipeline.py -m gpu -q -x -p no:cacheprovider -k "late or q19" > gpurun_out/r2zm_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2zm_pytest.log
for p in 1 0 1 0; do
  VD_LATE_PAIR=$p timeout 600 python bench.py --workload q19 --steps 20 --no-cpu-baseline 2>> gpurun_out/r2zm_bench.err | sed "s/^/pair$p /" >> gpurun_out/r2zm_q19.txt
done
VD_LATE_PAIR=1 timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_pipe_late -s 1 -c 1 -o gpurun_out/r2zm_prof_q19 -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline > gpurun_out/r2zm_ncu.log 2>&1
