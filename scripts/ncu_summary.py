#!/usr/bin/env python
"""Summarise ncu captures into profiles/ (committed evidence).

usage: python scripts/ncu_summary.py ROUND WORKLOAD=path.ncu-rep [...] [--launches path.csv]

Writes profiles/ncu_summary.json (per-workload dram bytes per launch, read by
bench.py's roofline.traffic) and profiles/<ROUND>_<workload>.md (key counters
of the `--set full` capture), plus profiles/<ROUND>_launches.md from a
`--metrics gpu__time_duration.sum` launch list.
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
PROF = os.path.join(ROOT, "profiles")

KEYS = [
    "gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
    "dram__throughput.avg.pct_of_peak_sustained_elapsed", "dram__bytes.sum.per_second",
    "lts__t_bytes.sum", "l1tex__t_bytes.sum", "sm__throughput.avg.pct_of_peak_sustained_elapsed",
    "smsp__issue_active.avg.pct_of_peak_sustained_active", "smsp__inst_executed.sum",
    "sm__warps_active.avg.pct_of_peak_sustained_active", "launch__registers_per_thread",
    "launch__grid_size", "launch__block_size", "launch__shared_mem_per_block_dynamic",
    "sm__cycles_elapsed.avg.per_second", "smsp__average_warps_issue_stalled_long_scoreboard_per_issue_active.ratio",
    "smsp__average_warps_issue_stalled_barrier_per_issue_active.ratio",
    "smsp__average_warps_issue_stalled_short_scoreboard_per_issue_active.ratio",
    "smsp__average_warps_issue_stalled_wait_per_issue_active.ratio",
    "smsp__average_warps_issue_stalled_mio_throttle_per_issue_active.ratio",
    "smsp__average_warps_issue_stalled_lg_throttle_per_issue_active.ratio",
    "smsp__average_warps_issue_stalled_branch_resolving_per_issue_active.ratio",
    "smsp__average_warps_issue_stalled_math_pipe_throttle_per_issue_active.ratio",
    "smsp__average_warps_issue_stalled_no_instruction_per_issue_active.ratio",
    "l1tex__data_pipe_lsu_wavefronts_mem_shared.sum",
    "lts__t_sectors.sum", "lts__t_sectors.sum.per_second", "lts__t_sectors_srcunit_tex_op_read.sum",
    "lts__throughput.avg.pct_of_peak_sustained_elapsed", "lts__t_sector_hit_rate.pct",
    "l1tex__t_sector_hit_rate.pct",
]

SCALE = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "Tbyte": 1e12}


def raw(rep):
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True, check=True)
    rows = list(csv.reader(io.StringIO(out.stdout)))
    hdr, units = rows[0], rows[1]
    res = []
    for r in rows[2:]:
        d = {}
        for h, u, v in zip(hdr, units, r):
            d[h] = (v, u)
        res.append(d)
    return res


def to_bytes(v, u):
    try:
        return float(v.replace(",", "")) * SCALE.get(u, 1)
    except ValueError:
        return None


def main():
    rnd = sys.argv[1]
    os.makedirs(PROF, exist_ok=True)
    summ_path = os.path.join(PROF, "ncu_summary.json")
    summ = json.load(open(summ_path)) if os.path.exists(summ_path) else {}
    args = sys.argv[2:]
    launches = None
    if "--launches" in args:
        i = args.index("--launches")
        launches = args[i + 1]
        args = args[:i] + args[i + 2:]
    for a in args:
        wl, rep = a.split("=", 1)
        kernels = raw(rep)
        lines = [f"# {rnd} ncu --set full: {wl}", "", f"source: `{os.path.basename(rep)}` (gpurun_out/, not committed)", ""]
        for k in kernels:
            name = k.get("Kernel Name", ("?", ""))[0]
            lines.append(f"## `{name[:120]}`")
            lines.append("")
            lines.append("| metric | unit | value |")
            lines.append("|---|---|---|")
            for key in KEYS:
                if key in k:
                    v, u = k[key]
                    lines.append(f"| {key} | {u} | {v} |")
            lines.append("")
        k0 = kernels[0]
        rd = to_bytes(*k0["dram__bytes_read.sum"])
        wr = to_bytes(*k0["dram__bytes_write.sum"])
        summ[wl] = {"kernel": k0.get("Kernel Name", ("?", ""))[0], "dram_bytes_read": rd, "dram_bytes_write": wr,
                    "dram_bytes_per_launch": (rd or 0) + (wr or 0), "round": rnd,
                    "duration": " ".join(k0["gpu__time_duration.sum"])}
        open(os.path.join(PROF, f"{rnd}_{wl}.md"), "w").write("\n".join(lines) + "\n")
    json.dump(summ, open(summ_path, "w"), indent=1)
    if launches:
        rows = list(csv.reader(open(launches)))
        hdr = None
        out = [f"# {rnd} launch list (`ncu --metrics gpu__time_duration.sum --clock-control none`)", "",
               "Cold-cache, serialised launches: compare shares, not absolutes.", "",
               "| # | kernel | grid | block | duration (ns) |", "|---|---|---|---|---|"]
        tot = {}
        for r in rows:
            if r and r[0] == "ID":
                hdr = r
                continue
            if hdr and len(r) == len(hdr):
                d = dict(zip(hdr, r))
                nm = d["Kernel Name"]
                out.append(f"| {d['ID']} | `{nm[:90]}` | {d['Grid Size']} | {d['Block Size']} | {d['Metric Value']} |")
                key = nm.split("(")[0]
                tot[key] = tot.get(key, 0) + float(d["Metric Value"].replace(",", ""))
        out += ["", "| kernel | total ns |", "|---|---|"]
        for k, v in sorted(tot.items(), key=lambda x: -x[1]):
            out.append(f"| `{k[:90]}` | {v:.0f} |")
        open(os.path.join(PROF, f"{rnd}_launches.md"), "w").write("\n".join(out) + "\n")


if __name__ == "__main__":
    main()
