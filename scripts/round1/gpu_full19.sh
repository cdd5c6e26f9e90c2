mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -p no:cacheprovider -k "q19" --durations=3 > gpurun_out/pytest_full19.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_full19.log
