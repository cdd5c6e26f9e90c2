# Round 2 (re-entry 3): final HEAD validation -- smoke, full GPU suite, bench lines of every workload
set -x
mkdir -p gpurun_out
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2zq_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/r2zq_smoke.log
timeout 3000 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/r2zq_pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/r2zq_pytest_gpu.log
timeout 600 python bench.py > gpurun_out/r2zq_bench_q1.json 2>> gpurun_out/r2zq_bench.err
for w in q6 q19 q9 q15 c1; do timeout 600 python bench.py --workload $w --no-cpu-baseline >> gpurun_out/r2zq_bench_all.jsonl 2>> gpurun_out/r2zq_bench.err; done
timeout 600 python bench.py --workload q6 --sf 100 --no-cpu-baseline >> gpurun_out/r2zq_bench_all.jsonl 2>> gpurun_out/r2zq_bench.err
for m in branch predicated; do timeout 300 python bench.py --workload selpos --selectivity 0.5 --sel-mode $m --no-cpu-baseline >> gpurun_out/r2zq_bench_all.jsonl 2>> gpurun_out/r2zq_bench.err; done
