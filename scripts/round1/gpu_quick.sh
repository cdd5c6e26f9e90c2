# Quick GPU iteration: focused parity tests + the affected benches.
set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -k "gather or layout" > gpurun_out/pytest_quick.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_quick.log
timeout 1200 python scripts/sweep.py fig14 > gpurun_out/sweep_fig14.jsonl 2>> gpurun_out/q_bench.err
