# Probes: random-lookup routes (L2 / DSMEM / local smem), write-only HBM
# bandwidth, and the selection benches + parity tests after a change.
set -x
mkdir -p gpurun_out
make -j16 > gpurun_out/make.log 2>&1
timeout 120 ./scripts/ubench_gather > gpurun_out/ubench_gather.jsonl 2>&1
timeout 120 python - > gpurun_out/wbw.txt 2>&1 <<'PY'
import torch
x = torch.empty(2 * 1024**3 // 4, dtype=torch.int32, device="cuda")
y = torch.empty(4 * 1024**3 // 4, dtype=torch.float32, device="cuda")
for name, f, nb in [("fill_2GiB", lambda: x.fill_(3), x.numel() * 4), ("sum_4GiB", lambda: y.sum(), y.numel() * 4)]:
    for _ in range(3): f()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize(); a.record()
    for _ in range(20): f()
    b.record(); torch.cuda.synchronize()
    ms = a.elapsed_time(b) / 20
    print(name, "%.4f ms" % ms, "%.1f GB/s" % (nb / ms / 1e6))
PY
timeout 900 python -m pytest tests/test_gpu_ops.py -m gpu -q -p no:cacheprovider -k "select or sel" > gpurun_out/pytest_sel.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_sel.log
for m in branch predicated; do timeout 300 python bench.py --workload selpos --selectivity 0.5 --sel-mode $m --no-cpu-baseline --no-e2e > gpurun_out/bench_selpos_$m.json 2>> gpurun_out/bench_misc.err; done
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_selpos.csv python bench.py --workload selpos --selectivity 0.5 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_launch.log 2>&1
