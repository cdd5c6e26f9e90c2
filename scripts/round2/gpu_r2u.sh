# Round 2: ncu of k_sel_stream (CNT=4) at s=1e-4 and s=0.5
mkdir -p gpurun_out
for s in 0.0001 0.5; do
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sel_stream -s 2 -c 1 -o gpurun_out/r2u_prof_s$s -f python bench.py --workload selpos --selectivity $s --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2u_ncu_$s.log 2>&1
done
