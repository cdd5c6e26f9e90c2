# Round 2 (re-entry 3): late fragment with 2 lead-qualified rows per thread per drain (Q19)
set -x
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_pipeline.py tests/test_gpu_fullsize.py -m gpu -q -x -p no:cacheprovider -k "late or q19 or fkj" > gpurun_out/r2zd_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2zd_pytest.log
for r in 2 1; do
  VD_LATE_R=$r timeout 600 python bench.py --workload q19 --steps 20 --no-cpu-baseline 2>> gpurun_out/r2zd_bench.err | sed "s/^/R$r /" >> gpurun_out/r2zd_q19.txt
done
for s in 0.001 0.01 0.05; do
  VD_LATE_R=2 timeout 600 python bench.py --workload fkjsel --selectivity $s --steps 20 --no-cpu-baseline 2>> gpurun_out/r2zd_bench.err | sed "s/^/R2 /" >> gpurun_out/r2zd_fkjsel.txt
  VD_LATE_R=1 timeout 600 python bench.py --workload fkjsel --selectivity $s --steps 20 --no-cpu-baseline 2>> gpurun_out/r2zd_bench.err | sed "s/^/R1 /" >> gpurun_out/r2zd_fkjsel.txt
done
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_pipe_late -s 1 -c 1 -o gpurun_out/r2zd_prof_q19 -f python bench.py --workload q19 --steps 1 --warmup 1 --no-cpu-baseline > gpurun_out/r2zd_ncu.log 2>&1
