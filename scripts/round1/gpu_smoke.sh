mkdir -p gpurun_out
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/smoke.log
timeout 900 python -m pytest tests/test_gpu_pipeline.py -m gpu -q -p no:cacheprovider -x -k "late or q19" > gpurun_out/pytest_late.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_late.log
