set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -k "select" > gpurun_out/pytest_sel.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_sel.log
for m in branch predicated; do timeout 300 python bench.py --workload selpos --selectivity 0.5 --sel-mode $m --no-cpu-baseline --no-e2e --steps 20 > gpurun_out/bench_selpos_$m.json 2>> gpurun_out/bench_misc.err; done
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -c 40 --csv --log-file gpurun_out/launches_selpos.csv python bench.py --workload selpos --selectivity 0.5 --steps 3 --warmup 3 > /dev/null 2>&1
