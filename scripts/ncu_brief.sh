ncu -i $1 --page raw --csv 2>/dev/null | python -c "
import csv,sys
r=list(csv.reader(sys.stdin))
h=r[0]
for row in r[2:]:
  for k,v in zip(h,row):
    if any(s in k for s in ['Kernel Name','gpu__time_duration.sum','dram__bytes_read.sum','dram__bytes_write.sum','issue_active.avg.pct','average_warps_issue_stalled','lts__t_sector_hit_rate','l1tex__data_pipe_lsu_wavefronts_mem_shared.sum','sm__inst_executed.sum','registers_per_thread','l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum']):
      if v and v not in ('0','0.000000') and not k.endswith('not_issued'):
        try:
          if 'stalled' in k and float(v) < 0.1: continue
        except: pass
        print(k,v)
"
