# Round 2: where the extra DRAM bytes of the late-materialisation fragments come from
set -x
mkdir -p gpurun_out
M=dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sectors_srcunit_tex_op_read.sum,lts__t_sectors_srcunit_tex_op_read_lookup_miss.sum,lts__t_sectors_srcunit_tex_op_red.sum,lts__t_sectors_srcunit_tex_op_red_lookup_miss.sum,lts__t_sectors_srcunit_tex_op_atom.sum,lts__t_sectors_op_read.sum,lts__t_sectors_op_write.sum,gpu__time_duration.sum
timeout 600 ncu --metrics $M --csv --log-file gpurun_out/r2e_ubench_gran.csv scripts/ubench_dram_gran > gpurun_out/r2e_ubench_gran.log 2>&1
scripts/ubench_dram_gran > gpurun_out/r2e_ubench_gran_timed.jsonl 2>&1
timeout 600 ncu --metrics $M --clock-control none -k regex:k_grp_fold_iv -s 2 -c 1 --csv --log-file gpurun_out/r2e_q15.csv python bench.py --workload q15 --steps 2 --warmup 2 --no-cpu-baseline > gpurun_out/r2e_q15.log 2>&1
timeout 600 ncu --metrics $M --clock-control none -k regex:k_pipe_late -s 2 -c 1 --csv --log-file gpurun_out/r2e_q19.csv python bench.py --workload q19 --steps 2 --warmup 2 --no-cpu-baseline --no-e2e > gpurun_out/r2e_q19.log 2>&1
