# Round 2 (re-entry 3): random 64-byte block read ceiling by target size
set -x
mkdir -p gpurun_out
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o scripts/ubench_random64 scripts/ubench_random64.cu
for g in 1 2 4 8 16; do timeout 300 ./scripts/ubench_random64 $g >> gpurun_out/r2zh_random64.jsonl 2>&1; done
