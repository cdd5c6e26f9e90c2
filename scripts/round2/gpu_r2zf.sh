# Round 2 (re-entry 3): random 64-byte block read ceiling; C1 launch list
set -x
mkdir -p gpurun_out
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o scripts/ubench_random64 scripts/ubench_random64.cu
timeout 300 ./scripts/ubench_random64 > gpurun_out/r2zf_random64.jsonl 2>&1
timeout 300 python bench.py --workload c1 --steps 50 --no-cpu-baseline > gpurun_out/r2zf_c1.json 2>> gpurun_out/r2zf_bench.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file gpurun_out/r2zf_c1_launches.csv python bench.py --workload c1 --steps 3 --warmup 3 --no-cpu-baseline > gpurun_out/r2zf_c1_ncu.log 2>&1
