# Round 2 (re-entry 3): late fast-round instances at 5 CTAs per SM (48 registers)
set -x
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_pipeline.py tests/test_gpu_fullsize.py -m gpu -q -x -p no:cacheprovider -k "late or q19 or fkj or star" > gpurun_out/r2zu_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2zu_pytest.log
for f in 1 0; do
  VD_LATE_FAST=$f timeout 600 python bench.py --workload q19 --steps 20 --no-cpu-baseline 2>> gpurun_out/r2zu_bench.err | sed "s/^/fast$f /" >> gpurun_out/r2zu_q19.txt
done
for s in 0.001 0.01 0.05 0.1; do
  timeout 600 python bench.py --workload fkjsel --selectivity $s --steps 20 --no-cpu-baseline 2>> gpurun_out/r2zu_bench.err >> gpurun_out/r2zu_fkjsel.txt
done
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_pipe_late -s 1 -c 1 -o gpurun_out/r2zu_prof_q19 -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline > gpurun_out/r2zu_ncu.log 2>&1
