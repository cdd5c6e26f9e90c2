set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -k "fold_scan" > gpurun_out/pytest_scan.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_scan.log
