set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_group.py -m gpu -q -p no:cacheprovider > gpurun_out/pytest_grp.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_grp.log
VD_GRP_GENERIC=1 timeout 900 python -m pytest tests/test_gpu_group.py -m gpu -q -p no:cacheprovider > gpurun_out/pytest_grp_generic.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_grp_generic.log
timeout 300 python bench.py --workload q15 --steps 30 > gpurun_out/bench_q15.json 2>> gpurun_out/bench_q15.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_grp_fold -s 1 -c 1 -o gpurun_out/prof_q15 -f python bench.py --workload q15 --steps 1 --warmup 1 > gpurun_out/ncu_q15.log 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 40 --csv --log-file gpurun_out/launches_q15.csv python bench.py --workload q15 --steps 2 --warmup 1 > /dev/null 2>&1
