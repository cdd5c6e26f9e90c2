# Round 2 (re-entry 3): k_sel_lag branching lane-owned fixed loop (VD_SEL_UNROLL) sweep
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_select_coop.py -m gpu -q -x -p no:cacheprovider -k "density" > gpurun_out/r2zr_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r2zr_pytest.log
for cfg in "320 1024" "640 1024" "640 160" "640 96" "640 64"; do set -- $cfg
  for s in 0.05 0.1 0.2 0.5 0.8; do
    VD_SEL_MID=$1 VD_SEL_UNROLL=$2 timeout 300 python bench.py --workload selpos --selectivity $s --steps 30 --no-cpu-baseline 2>> gpurun_out/r2zr_bench.err | sed "s/^/mid$1-unroll$2 /" >> gpurun_out/r2zr_selpos.txt
  done
done
