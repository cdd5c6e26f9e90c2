#!/usr/bin/env python
"""Selectivity sweeps on one GPU (runs bench.py per point; one JSON line each).

  python scripts/sweep.py fig1  > gpurun_out/sweep_fig1.jsonl   # C2: 1e9 f32 -> positions
  python scripts/sweep.py fig15 > gpurun_out/sweep_fig15.jsonl  # selective aggregation (select + FoldSum)
  python scripts/sweep.py fig16 > gpurun_out/sweep_fig16.jsonl  # selective FK join: branch / predicated / lookup
  python scripts/sweep.py fig14 > gpurun_out/sweep_fig14.jsonl  # multi-column lookups: single / separate / layout

Fig 1 and Fig 15: branching vs
predicated (cursor arithmetic) over selectivities 1..100 % (plus the Fig 15
range down to 0.01 %).  Then `python scripts/sweep.py table FILE...` renders
a markdown table for profiles/.
"""
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SEL = [0.0001, 0.001, 0.01, 0.05, 0.1, 0.2, 0.5, 0.8, 1.0]


def run(workload, s, mode, steps):
    cmd = [sys.executable, os.path.join(ROOT, "bench.py"), "--workload", workload, "--selectivity", str(s),
           "--sel-mode", mode, "--steps", str(steps), "--no-cpu-baseline", "--no-e2e"]
    out = subprocess.run(cmd, capture_output=True, text=True, timeout=600)
    line = out.stdout.strip().splitlines()[-1] if out.stdout.strip() else "{}"
    d = json.loads(line)
    d["_sel"] = s
    d["_mode"] = mode
    return d


def table(files):
    rows = []
    for f in files:
        for ln in open(f):
            if ln.strip():
                rows.append(json.loads(ln))
    print("| workload | selectivity | mode | ms | G rows/s | achieved GB/s | frac of measured |")
    print("|---|---|---|---|---|---|---|")
    for d in rows:
        if "roofline" not in d:
            continue
        print(f"| {d['config']['workload']} | {d['_sel']} | {d['_mode']} | {d['ms_per_step']:.3f} | "
              f"{d['value'] / 1e9:.1f} | {d['roofline']['achieved']:.0f} | {d['roofline']['frac']:.3f} |")


def fig14():
    """Fig 14: strategy x lookup pattern x target size."""
    for pattern in ["sequential", "random"]:
        for mb in [4, 1024]:
            for strat in ["single", "separate", "layout"]:
                cmd = [sys.executable, os.path.join(ROOT, "bench.py"), "--workload", "fig14", "--strategy", strat,
                       "--pattern", pattern, "--target-mb", str(mb), "--steps", "30"]
                out = subprocess.run(cmd, capture_output=True, text=True, timeout=600)
                line = out.stdout.strip().splitlines()[-1] if out.stdout.strip() else "{}"
                d = json.loads(line)
                d["_sel"] = f"{pattern} {mb}MB"
                d["_mode"] = strat
                print(json.dumps(d), flush=True)


def fig15m():
    """Fig 15 on B200 through the library's plans: selective
    aggregation sum(v2) where v1 between 0 and s over two 1e9-row f32
    columns -- fused branching / predicated, Break (predicate materialised),
    and the Vectorized plan (Materialize of per-chunk position lists)."""
    for s in SEL:
        for mat, chunk in (("none", 0), ("break", 0), ("chunks", 1024), ("chunks", 65536)):
            for mode in ("branch", "predicated"):
                cmd = [sys.executable, os.path.join(ROOT, "bench.py"), "--workload", "selagg", "--selectivity", str(s),
                       "--sel-mode", mode, "--materialize", mat, "--chunk", str(chunk), "--steps", "20",
                       "--no-cpu-baseline", "--no-e2e"]
                out = subprocess.run(cmd, capture_output=True, text=True, timeout=600)
                line = out.stdout.strip().splitlines()[-1] if out.stdout.strip() else "{}"
                d = json.loads(line)
                d["_sel"] = s
                d["_mode"] = f"{mode}/{mat}" + (f"/{chunk}" if mat == "chunks" else "")
                print(json.dumps(d), flush=True)


def main():
    what = sys.argv[1]
    if what == "fig15m":
        return fig15m()
    if what == "table":
        return table(sys.argv[2:])
    if what == "fig14":
        return fig14()
    workload = {"fig1": "selpos", "fig15": "select", "fig16": "fkjsel"}[what]
    modes = ["branch", "predicated", "lookup"] if what == "fig16" else ["branch", "predicated"]
    for s in SEL:
        for mode in modes:
            print(json.dumps(run(workload, s, mode, 30 if workload == "selpos" else 100)), flush=True)


if __name__ == "__main__":
    main()
