#!/usr/bin/env python
"""Benchmark of the Voodoo hot path on B200 (BASELINE.json metric).

Default: TPC-H Q1 at SF100 (600 M lineitem rows, 22.8 GB of columns),
row-range partitioned across the N GPUs of one node (one process per GPU,
launched by torch.distributed.run for N > 1).  A step is one pass of the
fused Q1 fragment over the whole table: predicate (a2), virtual
Partition/Scatter (a5), grouped folds (a6/a7), the hierarchical fold down to
one partials vector per GPU (a8) and, for N > 1, the NCCL all-gather of
those partials (the cross-GPU exchange step).  Inputs are generated in HBM
before the timed region (excluded) and are far larger
than the 126 MB L2, so no flush is needed between steps.

Prints ONE JSON line on rank 0 (the driver contract), with `roofline`,
`cpu_baseline` (the oracle on a bounded sample), `clocks`, `e2e` and
`gpu_launches`.  `--impl reference` times the CPU oracle (the tier's
reference arm) on the same config and metric instead.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

METRIC = "rows/s and achieved HBM GB/s (% of peak) for TPC-H Q1/Q6 at 1/2/4/8 B200"

# Algorithmic bytes per row: every
# column each query reads, once.
BYTES_PER_ROW = {"q1": 4 + 1 + 1 + 4 * 8, "q6": 4 + 3 * 8, "select": 4, "selpos": 4, "c1": 4, "selagg": 8,
                 "q19": 4 + 3 * 8 + 1 + 1, "q9": 4 + 4 + 2 * 8, "fkjsel": 4 + 4, "q15": 24}
L2_CAP_BYTES_PER_CLK = 6300  # B300_MICROARCH.md "LTS throughput cap" (full chip)


def parse():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=None)
    ap.add_argument("--warmup", type=int, default=5)
    ap.add_argument("--impl", default="voodoo", choices=["voodoo", "reference"])
    ap.add_argument("--workload", default="q1",
                    choices=["q1", "q6", "select", "selagg", "selpos", "q19", "q9", "fkjsel", "fig14", "q15",
                             "c1"])
    ap.add_argument("--materialize", default="none", choices=["none", "break", "chunks"],
                    help="selagg/q6/q1: the pipeline plan -- fused, Break (predicate materialised, Fig 8) or "
                         "Materialize of per-chunk position lists (Fig 15 'Vectorized')")
    ap.add_argument("--chunk", type=int, default=0, help="--materialize chunks: rows per chunk (0 = 1024)")
    ap.add_argument("--sf", type=float, default=None, help="scale factor (default: q1 100, q6 10, fkj 100)")
    ap.add_argument("--sel-mode", default="branch", choices=["branch", "predicated", "lookup"])
    ap.add_argument("--selectivity", type=float, default=0.5, help="select workload: fraction selected")
    ap.add_argument("--rows", type=int, default=None, help="select workload: rows (default 1e9)")
    ap.add_argument("--generic", action="store_true", help="force the generic fragment")
    ap.add_argument("--strategy", default="layout", choices=["single", "separate", "layout"],
                    help="fig14: Single Loop / Separate Loops / Layout Transform (P:L1156-1193)")
    ap.add_argument("--pattern", default="random", choices=["random", "sequential"], help="fig14 lookup pattern")
    ap.add_argument("--target-mb", type=int, default=1024, help="fig14 target table size (two int32 columns)")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--cpu-seconds", type=float, default=10.0)
    ap.add_argument("--seed", type=int, default=0x5EEDC0DE)
    ap.add_argument("--no-graph", action="store_true", help="N > 1: launch eagerly instead of CUDA graphs")
    ap.add_argument("--graph", action="store_true", help="replay the step as CUDA graphs at N = 1 too")
    ap.add_argument("--grouping", default="direct", choices=["direct", "hash"],
                    help="q15: identity-hashed table over min..max (vd_group_fold) or open addressing "
                         "(vd_hash_group_fold)")
    ap.add_argument("--dist-backend", default="nccl", choices=["nccl", "gloo"],
                    help="process-group backend for N > 1 (gloo: test mode, ranks may share a GPU)")
    return ap.parse_args()


def default_sf(w):
    return {"q15": 100.0, "q1": 100.0, "q6": 10.0, "q19": 100.0, "q9": 100.0, "select": 0.0, "selpos": 0.0, "fkjsel": 0.0,
            "selagg": 0.0, "c1": 0.0, "fig14": 0.0}[w]


# ---------------------------------------------------------------------------
# measured peaks (driver-written)
# ---------------------------------------------------------------------------
def hbm_peak():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            return float(json.load(f)["hbm_gbs"]), "measured"
    except Exception:
        return 6650.0, "fallback"


NOMINAL_HBM_GBS = 8000.0  # B200 HBM3e nominal (report beside the measured peak)


def hbm_roofline(achieved, kernel, kernel_ms, traffic=None, **extra):
    """`roofline` object for an HBM-bound kernel: achieved algorithmic GB/s
    against the measured copy peak (MEASURED_PEAKS.json) and, beside it, the
    nominal 8 TB/s."""
    peak, kind = hbm_peak()
    return {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s", "frac": achieved / peak,
            "peak_kind": kind, "peak_nominal": NOMINAL_HBM_GBS, "frac_nominal": achieved / NOMINAL_HBM_GBS,
            "traffic": traffic, "kernel": kernel, "kernel_ms": kernel_ms, **extra}


def ncu_traffic(workload, world=1):
    """dram bytes per launch of the dominant kernel from the committed
    `ncu --set full` summary (profiles/ncu_summary.json), else None.  The
    capture is of the single-GPU launch; a rank of an N-GPU run scans a
    1/N row range, so its per-launch traffic is the capture's / N (the
    streamed columns dominate; replicated dimension tables are a small
    constant)."""
    try:
        with open(os.path.join(ROOT, "profiles", "ncu_summary.json")) as f:
            d = json.load(f)
        t = d.get(workload, {}).get("dram_bytes_per_launch")
        return None if t is None else t / max(world, 1)
    except Exception:
        return None


# ---------------------------------------------------------------------------
# clocks sampled during the timed region
# ---------------------------------------------------------------------------
class ClockSampler:
    FIELDS = ("index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active,"
              "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
              "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, dev):
        self.dev = dev
        self.proc = None
        self.lines = []
        self.t = None

    def start(self):
        try:
            self.proc = subprocess.Popen(["nvidia-smi", f"--query-gpu={self.FIELDS}", "--format=csv,noheader,nounits",
                                          "-lms", "100", "-i", str(self.dev)], stdout=subprocess.PIPE,
                                         stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
        except Exception:
            self.proc = None

    def _read(self):
        for line in self.proc.stdout:
            self.lines.append(line.strip())

    def stop(self):
        if self.proc is None:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvidia-smi unavailable"]}
        self.proc.terminate()
        try:
            self.proc.wait(timeout=5)
        except Exception:
            self.proc.kill()
        if self.t:
            self.t.join(timeout=2)
        sm, mx, reasons = [], [], set()
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        for ln in self.lines:
            p = [x.strip() for x in ln.split(",")]
            if len(p) < 9:
                continue
            try:
                sm.append(float(p[1]))
                mx.append(float(p[2]))
            except ValueError:
                continue
            for nm, v in zip(names, p[5:9]):
                if v.lower() == "active":
                    reasons.add(nm)
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": sorted(reasons), "samples": len(sm)}


# ---------------------------------------------------------------------------
# CPU oracle baseline (bounded sample)
# ---------------------------------------------------------------------------
def host_info():
    """CPU model string and host RAM (SURVEY §8(d) timing protocol)."""
    model, ram = None, None
    try:
        with open("/proc/cpuinfo") as f:
            for ln in f:
                if ln.startswith("model name"):
                    model = ln.split(":", 1)[1].strip()
                    break
    except OSError:
        pass
    try:
        with open("/proc/meminfo") as f:
            for ln in f:
                if ln.startswith("MemTotal"):
                    ram = round(int(ln.split()[1]) / 2**20, 1)
                    break
    except OSError:
        pass
    return {"cpu_model": model, "host_ram_gib": ram, "hardware_concurrency": os.cpu_count()}


def oracle_task(workload, sf, seed, sel_t):
    """(make(row0, m) -> inputs, run(inputs) -> handle, extract(handle) ->
    partial, merge(a, b), what): the oracle program of each workload over one
    row range.  Only `run` is timed (extracting results into Python objects
    is not the oracle's work).  Partials decompose over row ranges (pin P8),
    so a partitioned run merges them."""
    import numpy as np

    import gen
    import oracle
    from oracle import programs

    def add_dict(a, b):
        out = dict(a)
        for k, v in b.items():
            out[k] = [x + y for x, y in zip(out[k], v)] if k in out else list(v)
        return out

    def add_tuple(a, b):
        return tuple(x + y for x, y in zip(a, b))

    def ident(x):
        return x

    def head(p, name):
        v, e = p.get_arrays(name)
        return v[:1][~e[:1]].tolist()[0] if v.size and not e[0] else 0

    if workload in ("select", "selpos"):
        def make(row0, m):
            return gen.host(gen.F32_UNIFORM, m, row0, seed=seed)
        if workload == "select":
            def run(v):
                p = oracle.Program()
                p.set("input.val", v)
                return p.run(programs.SELECT_SUM.format(intent=v.size, t=float(np.float32(sel_t)).hex()))

            def extract(p):
                return (float(head(p, "totalSum")), int(head(p, "count")))
            return make, run, extract, add_tuple, "literal Voodoo interpreter, SELECT_SUM program (Fig 8 shape)"

        def run(v):
            return (oracle.select_f32(v, float(np.float32(sel_t)), "lt")[1],)
        return make, run, ident, add_tuple, "brute-force selection loop -> int32 positions (oracle/tpch_oracle.cpp)"

    names = {"q1": plans_cols("Q1_COLS"), "q6": plans_cols("Q6_COLS"), "q15": ["l_shipdate", "l_suppkey",
             "l_extendedprice", "l_discount"]}.get(workload, list(gen.LINEITEM_COLS))

    def make(row0, m):
        return {k: gen.host(gen.LINEITEM_COLS[k], m, row0, sf=sf, seed=seed) for k in names}

    if workload == "q1":
        def run(li):
            p = oracle.Program()
            for k, v in li.items():
                p.set("lineitem." + k, v)
            return p.run(programs.Q1.format(ship_max_p1=10472))

        def extract(p):
            keys, ke = p.get_arrays("o_key")
            sel = ~ke
            outs = [p.get_arrays(o)[0][sel] for o in programs.Q1_OUTPUTS]
            return {int(k): [int(o[j]) for o in outs] for j, k in enumerate(keys[sel].tolist())}
        return make, run, extract, add_dict, "literal Voodoo interpreter, Q1 program (Fig 10/11 shape)"
    if workload == "q6":
        def run(li):
            p = oracle.Program()
            for k, v in li.items():
                p.set("lineitem." + k, v)
            return p.run(programs.Q6.format(intent=1 << 30, d0m1=8765, d1=9131, dlom1=4, dhip1=8, qmax=2400))

        def extract(p):
            return (int(head(p, "revenue")), int(head(p, "count")))
        return make, run, extract, add_tuple, "literal Voodoo interpreter, Q6 program (Fig 8 shape)"
    if workload == "q15":
        def run(li):
            return {k: list(v) for k, v in oracle.q15(li).items()}
        return make, run, ident, add_dict, "brute-force Q15 revenue-view loop (oracle/tpch_oracle.cpp)"
    # FK joins (C5): the brute-force join loop over the replicated dimension tables
    part = {k: gen.host(c, gen.part_rows(sf), sf=sf, seed=seed) for k, c in gen.PART_COLS.items()}
    supp = {k: gen.host(c, gen.supplier_rows(sf), sf=sf, seed=seed) for k, c in gen.SUPPLIER_COLS.items()}
    variant = 0 if workload == "q19" else 1

    def run(li):
        return {k: list(v) for k, v in oracle.fkj(variant, li, part, supp).items()}
    return make, run, ident, add_dict, f"brute-force {workload.upper()}-style FK join loop (oracle/tpch_oracle.cpp)"


def plans_cols(name):
    from paper_journals_pvldb_pirkmzm16_b200 import plans
    return list(getattr(plans, name))


def cpu_baseline(workload, sf, seed, budget_s, sel_t=0.5, n_total=None, partitioned=True):
    """Time the oracle as it stands on a bounded sample of the workload:
    single-threaded over row chunks until ~budget_s of CPU work, then (SURVEY
    §8(d)) the same rows partitioned over N = hardware_concurrency threads,
    thread i interpreting rows [i*S/N, (i+1)*S/N) (the Fig 3 control vector,
    P:L241-250) and the partials merged.  Input generation is excluded."""
    import concurrent.futures as cf

    import gen

    if workload == "fkjsel":
        return None
    make, run, extract, merge, what = oracle_task(workload, sf, seed, sel_t)
    chunk = 1 << 19
    if n_total is None:
        n_total = gen.lineitem_rows(sf) if workload not in ("select", "selpos") else 10**9
    rows_done, t_total, row0, res1 = 0, 0.0, 0, None
    while t_total < budget_s and row0 < n_total:
        m = min(chunk, n_total - row0)
        x = make(row0, m)
        t0 = time.perf_counter()
        h = run(x)
        t_total += time.perf_counter() - t0
        r = extract(h)
        del h
        res1 = r if res1 is None else merge(res1, r)
        rows_done += m
        row0 += m
    out = {"value": rows_done / t_total, "unit": "rows/s", "cores": 1, "kind": "oracle",
           "sample": f"{rows_done} rows of the {workload} workload (rows 0..{rows_done - 1}, chunks of {chunk}), "
                     f"{what}, {t_total:.1f} s single-threaded",
           "seconds": t_total, **host_info()}
    if partitioned and rows_done > 0:
        N = os.cpu_count() or 1
        bounds = [(i * rows_done // N, (i + 1) * rows_done // N) for i in range(N)]
        sub = 1 << 17
        work = [[make(a0, min(sub, b - a0)) for a0 in range(a, b, sub)] for a, b in bounds]

        def thread(items):  # ctypes releases the GIL inside the C oracle
            return [run(x) for x in items]

        t0 = time.perf_counter()
        with cf.ThreadPoolExecutor(N) as ex:
            handles = list(ex.map(thread, work))
        dt = time.perf_counter() - t0
        resN = None
        for hs in handles:
            for h in hs:
                r = extract(h)
                resN = r if resN is None else merge(resN, r)
        del handles, work
        same = resN == res1 if workload != "select" else (
            abs(resN[0] - res1[0]) <= 1e-9 * abs(res1[0]) and resN[1] == res1[1])
        out["partitioned"] = {"value": rows_done / dt, "unit": "rows/s", "threads": N, "seconds": dt,
                              "merged_equals_single_thread": bool(same),
                              "sample": f"the same {rows_done} rows, thread i -> rows [i*S/N, (i+1)*S/N) "
                                        f"(Fig 3 control vector), sub-chunks of {sub}, partials merged"}
    return out


# ---------------------------------------------------------------------------
# the GPU arm
# ---------------------------------------------------------------------------
def main():
    args = parse()
    rank = int(os.environ.get("RANK", "0"))
    world = int(os.environ.get("WORLD_SIZE", "1"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    sf = args.sf if args.sf is not None else default_sf(args.workload)

    if args.impl == "reference":
        return reference_arm(args, rank, world, sf)
    if args.workload == "selpos":
        return selpos_main(args, rank, world, local)
    if args.workload == "fig14":
        return fig14_main(args, rank, world, local)
    if args.workload == "q15":
        return q15_main(args, rank, world, local, sf)
    if args.workload == "c1":
        return c1_main(args, rank, world, local)

    import torch
    import torch.distributed as dist

    import gen
    from paper_journals_pvldb_pirkmzm16_b200 import plans, vd

    ndev = torch.cuda.device_count()
    torch.cuda.set_device(local % ndev)
    dev = torch.device("cuda", local % ndev)
    comm = Comm(world, args.dist_backend, dev)
    stream = torch.cuda.current_stream()

    w = args.workload
    n_total = workload_rows(args, w, sf)
    a, b = rank * n_total // world, (rank + 1) * n_total // world
    n = b - a
    sel_mode = {"branch": vd.VD_SEL_BRANCH, "predicated": vd.VD_SEL_PREDICATED,
                "lookup": vd.VD_SEL_PREDICATED_LOOKUP}[args.sel_mode]

    # ---- a1: columns generated in HBM (row range [a, b)), min/max via vd folds
    def make(col, length, row0, sfv=sf, **kw):
        t = torch.empty(length, dtype=getattr(torch, _dt(col)), device=dev)
        gen.device(col, t.data_ptr(), length, row0, sf=sfv, seed=args.seed, stream=stream.cuda_stream, **kw)
        return t

    def meta(t):
        return vd.describe(t, stream=stream)

    dims, dim_views, cols = [], [], []
    if w == "q1":
        names, plan = plans.Q1_COLS, plans.q1(sel_mode, force_generic=args.generic)
    elif w == "q6":
        names, plan = plans.Q6_COLS, plans.q6(sel_mode, force_generic=args.generic)
    elif w == "q19":
        names = plans.Q19_COLS
        plan = plans.q19({"brand": {s: i for i, s in enumerate(gen.BRAND)},
                          "container": {s: i for i, s in enumerate(gen.CONTAINER)},
                          "shipmode": {s: i for i, s in enumerate(gen.SHIPMODE)},
                          "shipinstruct": {s: i for i, s in enumerate(gen.SHIPINSTRUCT)}}, sel_mode,
                         force_generic=args.generic)
        for d in plans.Q19_DIMS:
            dims.append(make(gen.PART_COLS[d], gen.part_rows(sf), 0))
    elif w == "q9":
        names, plan = plans.Q9_COLS, plans.q9(sel_mode, force_generic=args.generic)
        for d in plans.Q9_DIMS:
            dims.append(make(gen.SUPPLIER_COLS[d], gen.supplier_rows(sf), 0))
    elif w == "fkjsel":
        # Fig 16: fact(fk, v) x target(v) through fk - 1, v < threshold, sum(target.v)
        m = plans.FKJSEL_TARGET_ROWS
        names = ["fk", "v"]
        thr = int(round(args.selectivity * plans.FKJSEL_VMAX))
        plan = plans.fkjsel(thr, sel_mode, force_generic=args.generic)
        t = torch.empty(m, dtype=torch.int64, device=dev)
        gen.device(gen.I64_UNIFORM, t.data_ptr(), m, 0, seed=args.seed + 2, p0=0, p1=10**6, stream=stream.cuda_stream)
        dims.append(t)
    elif w == "selagg":
        # Fig 15: sum(v2) where v1 between 0 and s, two f32 columns
        names = ["v1", "v2"]
        plan = plans.selagg(0.0, float(__import__("numpy").float32(args.selectivity)), sel_mode)
    else:
        names = ["v"]
        plan = plans.selsum(float(__import__("numpy").float32(args.selectivity)), sel_mode,
                            force_generic=args.generic)
    mat = {"none": vd.VD_MAT_NONE, "break": vd.VD_MAT_BREAK, "chunks": vd.VD_MAT_CHUNKS}[args.materialize]
    plan.materialize, plan.mat_chunk = mat, args.chunk
    for nm in names:
        if w == "fkjsel":
            c = torch.empty(n, dtype=torch.int32, device=dev)
            if nm == "fk":
                gen.device(gen.I32_UNIFORM, c.data_ptr(), n, a, seed=args.seed, p0=1, p1=plans.FKJSEL_TARGET_ROWS,
                           stream=stream.cuda_stream)
            else:
                gen.device(gen.I32_UNIFORM, c.data_ptr(), n, a, seed=args.seed + 1, p0=0, p1=plans.FKJSEL_VMAX - 1,
                           stream=stream.cuda_stream)
            cols.append(c)
            continue
        if nm in ("v", "v1", "v2"):
            t = torch.empty(n, dtype=torch.float32, device=dev)
            gen.device(gen.F32_UNIFORM, t.data_ptr(), n, a, seed=args.seed + (nm == "v2"), stream=stream.cuda_stream)
            cols.append(t)
            continue
        cols.append(make(gen.LINEITEM_COLS[nm], n, a))
    torch.cuda.synchronize()
    views = [meta(t) for t in cols]
    dim_views = [meta(t) for t in dims]
    torch.cuda.synchronize()

    pbytes = vd.partials_bytes(plan)
    out = torch.empty(pbytes, dtype=torch.uint8, device=dev)
    ws = vd.alloc_ws(vd.workspace_bytes(vd.VD_OP_PIPELINE, n, None, plan), dev)
    gathered = torch.empty(pbytes * world, dtype=torch.uint8, device=dev) if world > 1 else out
    result = vd.DeviceResult(plan, dev)

    # A step: the fused fragment over this rank's rows (a2-a9), then the
    # cross-GPU step (all-gather of the partials, N > 1) and the device merge
    # + Fig 11 compaction into a vd_result -- the query's answer is on the
    # device when the step ends (no host round trip).
    def pipe():
        vd.run_pipeline(plan, views, n, dim_views, out=out, ws=ws, stream=stream)

    def exchange():
        comm.all_gather(out, gathered)
        vd.merge_partials_device(plan, views, dim_views, gathered, world, result, stream=stream)

    steps = args.steps if args.steps is not None else (300 if w in ("q1", "q19", "q9") else 1000)
    for _ in range(max(args.warmup, 0)):
        pipe()
        launches_per_step = vd.last_launch_count()
        exchange()
        launches_per_step += vd.last_launch_count()
    frag = vd.last_fragment()
    torch.cuda.synchronize()
    # N > 1: the two halves of the step replayed as CUDA graphs (launch
    # latency off the critical path of ~0.4 ms shards); N = 1 runs eagerly
    graphs = None
    if ((world > 1 and comm.backend == "nccl") or args.graph) and not args.no_graph:
        try:
            g1, g2 = torch.cuda.CUDAGraph(), torch.cuda.CUDAGraph()
            side = torch.cuda.Stream(device=dev)
            side.wait_stream(stream)
            with torch.cuda.stream(side):
                with torch.cuda.graph(g1, stream=side):
                    vd.run_pipeline(plan, views, n, dim_views, out=out, ws=ws, stream=side)
                with torch.cuda.graph(g2, stream=side):
                    comm.all_gather(out, gathered)
                    vd.merge_partials_device(plan, views, dim_views, gathered, world, result, stream=side)
            stream.wait_stream(side)
            torch.cuda.synchronize()
            graphs = (g1, g2)
            pipe = g1.replay  # noqa: F811
            exchange = g2.replay  # noqa: F811
            for _ in range(2):
                pipe()
                exchange()
            torch.cuda.synchronize()
        except Exception as e:  # capture unsupported here: stay eager, say so
            graphs = f"eager (capture failed: {type(e).__name__}: {e})"[:200]

    # ---- timed region --------------------------------------------------------
    clocks = ClockSampler(local)
    clocks.start()
    time.sleep(0.3)
    comm.barrier()
    torch.cuda.synchronize()
    ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)) for _ in range(steps)]
    t_start = torch.cuda.Event(enable_timing=True)
    t_end = torch.cuda.Event(enable_timing=True)
    wall0 = time.perf_counter()
    t_start.record(stream)
    for i in range(steps):
        ev[i][0].record(stream)
        pipe()
        ev[i][1].record(stream)
        exchange()
    t_end.record(stream)
    torch.cuda.synchronize()
    comm.barrier()
    wall = time.perf_counter() - wall0
    clk = clocks.stop()
    elapsed_ms = t_start.elapsed_time(t_end)
    kernel_ms = sum(s.elapsed_time(e) for s, e in ev) / steps
    elapsed_ms, kernel_ms = comm.max([elapsed_ms, kernel_ms])
    ms_per_step = elapsed_ms / steps

    # the step's answer: the device vd_result (merged + compacted on the GPU)
    fl = [w in ("select", "selagg")] + [False] * 8
    result_dev = result
    result = result_dev.decode(plan, float_aggs=fl)
    if world > 1:  # cross-check against the host merge of the gathered partials
        parts = [gathered[r * pbytes:(r + 1) * pbytes].cpu().numpy().tobytes() for r in range(world)]
        assert vd.merge_partials(plan, views, dim_views, parts, float_aggs=fl) == result

    # ---- e2e: host buffers in, result out, through the public API -------------
    e2e = None
    if not args.no_e2e:
        e2e = e2e_measure(args, torch, vd, plan, cols, views, dims, dim_views, n, dev, stream, world, comm, pbytes)

    peak, peak_kind = hbm_peak()
    bpr = BYTES_PER_ROW[w]
    alg_bytes = n * bpr
    extra = {}
    if w == "fkjsel":
        # reading A33: a lookup into a table larger than L2 (128 Mi x 8 B =
        # 1 GiB) moves one 64-byte HBM block; branching and predicated-lookup
        # plans look up the qualifying rows only (the lookup plan sends the
        # rest to the hot slot 0), predicated aggregation looks up every row
        sel_rows = int(next(iter(result.values()))[-1]) if result else 0
        looked_up = n if args.sel_mode == "predicated" else sel_rows // max(world, 1)
        alg_bytes = n * bpr + 64 * looked_up
        extra = {"bytes_per_row_dense": bpr, "lookups": looked_up, "lookup_granule_bytes": 64}
        if frag == "late":
            # late materialisation (A31/A33/A34): fact.v in full, of fact.fk
            # the 64-byte blocks holding a qualifying row, 64 B per lookup
            thr = int(round(args.selectivity * plans.FKJSEL_VMAX))
            mask = cols[1] < thr
            r = 64 // cols[0].element_size()
            full = n // r * r
            fk_blocks = int(mask[:full].view(-1, r).any(1).sum().item()) + int(bool(mask[full:].any().item()))
            looked_up = int(mask.sum().item())
            alg_bytes = n * cols[1].element_size() + 64 * fk_blocks + 64 * looked_up
            extra = {"bytes_per_row_dense": bpr, "lookups": looked_up, "lookup_granule_bytes": 64,
                     "fk_blocks": fk_blocks}
            del mask
    elif w == "q19" and frag == "late":
        # late-materialisation fragment, readings A31/A33: the lead columns
        # (l_shipmode, l_shipinstruct: the u8 terms every conjunction shares)
        # in full; of l_partkey / l_quantity the 64-byte blocks holding a
        # lead-qualified row, of l_extendedprice / l_discount those holding a
        # qualifying row; the part table (120 MB at SF100, L2-sized) once;
        # the lookups themselves are L2 sectors (roofline.l2)
        alg_bytes, extra = q19_late_bytes(plan, cols, dims, result, clk, kernel_ms)
    elif w in ("q9", "q19"):
        # the dimension lookups hit L2 (supplier 1 MB; part 120 MB at SF100):
        # the second bound is L2 slice throughput, one 32-byte sector per
        # lookup on top of the streamed sectors
        nlook = n if w == "q9" else None
        if nlook is not None:
            sectors = n * bpr / 32 + nlook
            clk_ghz = (clk or {}).get("sm_mhz") or 1965.0
            cap = L2_CAP_BYTES_PER_CLK * clk_ghz / 1e3 / 32  # sectors per ns
            ach = sectors / (kernel_ms * 1e6)
            extra = {"l2": {"bound": "l2", "sectors_per_row": bpr / 32 + 1, "achieved": ach, "peak": cap,
                            "unit": "sectors/ns", "frac": ach / cap,
                            "peak_kind": "guide: B300-measured LTS cap 6300 B/clk x SM clock (B300_MICROARCH.md)"}}
    achieved = alg_bytes / (kernel_ms * 1e-3) / 1e9  # per GPU, dominant-kernel duration
    rows_per_s = n_total / (ms_per_step * 1e-3)
    line = {
        "metric": METRIC,
        "value": rows_per_s,
        "unit": "rows/s",
        "n_gpus": world,
        "steps": steps,
        "warmup": args.warmup,
        "ms_per_step": ms_per_step,
        "higher_is_better": True,
        "scaling": "strong",
        "vs_baseline": None,
        "dtype": "f32/f64" if w in ("select", "selagg") else "int64",
        "data": "synthetic (dbgen-shaped, counter-based generator gen/vd_gen.h, generated in HBM)",
        "config": bench_config(args, w, sf, world),
        "fragment": "generic" if args.generic else frag,
        "cuda_graphs": ("pipeline + (all-gather, merge)" if isinstance(graphs, tuple) else graphs),
        "hbm_gbs": achieved,
        "roofline": hbm_roofline(
            achieved, "k_pipe_q1_tma" if w == "q1" and not args.generic else "vd_run_pipeline", kernel_ms,
            ncu_traffic(f"fkjsel_s{args.selectivity:g}_{args.sel_mode}" if w == "fkjsel" else w, world),
            bytes_per_row=alg_bytes / n if n else bpr, **extra),
        "clocks": clk,
        "e2e": e2e,
        "gpu_launches": launches_per_step * steps,
        "result": {str(k): [str(x) for x in v] for k, v in list(result.items())[:8]},
        "result_groups": len(result),
        "result_digest": __import__("hashlib").sha256(repr(sorted(result.items())).encode()).hexdigest()[:16],
        "wall_s": wall,
    }
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        cb = cpu_baseline(w, sf, args.seed, args.cpu_seconds, args.selectivity, n_total)
        if cb is not None:
            line["cpu_baseline"] = cb
    if rank == 0:
        print(json.dumps(line), flush=True)
    comm.close()


SEL_KERNELS = {"sel_lag": "k_sel_lag (one cooperative launch, lagged decode)",
               "sel_coop": "k_sel_coop (one cooperative launch, one grid barrier)",
               "sel_bitmap": "k_sel_bits + k_scan_i32 + k_sel_total + k_sel_write",
               "sel_lookback": "k_sel_lookback"}


def selpos_main(args, rank, world, local):
    """C2 (Fig 1 sweep point): select v < t over 1e9 f32 -> int32 positions,
    branching or predicated (vd_select_*).  Algorithmic bytes: 4 B/row read +
    4 B per selected row written."""
    import numpy as np
    import torch
    import torch.distributed as dist

    import gen
    from paper_journals_pvldb_pirkmzm16_b200 import vd

    ndev = torch.cuda.device_count()
    torch.cuda.set_device(local % ndev)
    dev = torch.device("cuda", local % ndev)
    comm = Comm(world, args.dist_backend, dev)
    stream = torch.cuda.current_stream()
    n_total = args.rows or 10**9
    a, b = rank * n_total // world, (rank + 1) * n_total // world
    n = b - a
    v = torch.empty(n, dtype=torch.float32, device=dev)
    gen.device(gen.F32_UNIFORM, v.data_ptr(), n, a, seed=args.seed, stream=stream.cuda_stream)
    t = float(np.float32(args.selectivity))
    pos = torch.empty(n, dtype=torch.int32, device=dev)
    cnt = torch.zeros(1, dtype=torch.int64, device=dev)
    ws = vd.alloc_ws(vd.workspace_bytes(vd.VD_OP_SELECT, n), dev)
    fn = vd.select_predicated if args.sel_mode == "predicated" else vd.select_branch
    cols = [vd.column(v)]
    p = vd.pred([[(0, "<", t)]])

    def step():
        fn(cols, n, p, out_pos=pos, out_count=cnt, ws=ws, stream=stream)

    for _ in range(max(args.warmup, 3)):
        step()
    lps = vd.last_launch_count()
    frag = vd.last_fragment()
    torch.cuda.synchronize()
    steps = args.steps or 200
    clocks = ClockSampler(local)
    clocks.start()
    time.sleep(0.3)
    comm.barrier()
    torch.cuda.synchronize()
    ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)) for _ in range(steps)]
    for i in range(steps):
        ev[i][0].record(stream)
        step()
        ev[i][1].record(stream)
    torch.cuda.synchronize()
    clk = clocks.stop()
    ms = sum(s.elapsed_time(e) for s, e in ev) / steps
    ms = comm.max([ms])[0]
    c = int(cnt.item())
    peak, kind = hbm_peak()
    alg = (4 * n + 4 * c) / (ms * 1e-3) / 1e9
    line = {"metric": METRIC, "value": n_total / (ms * 1e-3), "unit": "rows/s", "n_gpus": world, "steps": steps,
            "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True, "scaling": "strong",
            "vs_baseline": None, "dtype": "f32", "data": "synthetic (f32 U[0,1), gen/vd_gen.h)",
            "config": bench_config(args, "selpos", 0.0, world),
            "selected": c, "achieved_selectivity": c / n,
            "roofline": hbm_roofline(alg, SEL_KERNELS.get(frag, frag), ms,
                                     ncu_traffic(f"selpos_s{args.selectivity:g}_{args.sel_mode}", world)),
            "clocks": clk, "e2e": None, "gpu_launches": lps * steps}
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        cb = cpu_baseline("selpos", 0.0, args.seed, args.cpu_seconds, args.selectivity, n_total)
        if cb is not None:
            line["cpu_baseline"] = cb
    if rank == 0:
        print(json.dumps(line), flush=True)
    comm.close()


def c1_main(args, rank, world, local):
    """C1 (BASELINE.json configs[0]): 2^20 f32 U[0,1), v < 0.5, branching vs
    predicated: the position list (vd_select_*, Fig 1) plus the FoldSum of
    the selected values (the fused selective-sum fragment, Fig 8/15).  The
    4 MiB input is L2-resident by design, so the HBM roofline does not
    apply: per-call microseconds are reported warm (back to back) and cold
    (each call after a 512 MB write that evicts L2), on the launching stream
    with CUDA events around CUDA-graph replays of each call (so the events
    time GPU work, not Python marshalling).  A step = positions + sum, both
    modes reported; the
    line's value is the warm branching step.  Each rank runs an independent
    replica (C1 does not shard: 'replicas only')."""
    import numpy as np
    import torch

    import gen
    import oracle
    from paper_journals_pvldb_pirkmzm16_b200 import plans, vd

    ndev = torch.cuda.device_count()
    torch.cuda.set_device(local % ndev)
    dev = torch.device("cuda", local % ndev)
    comm = Comm(world, args.dist_backend, dev)
    stream = torch.cuda.current_stream()
    n = args.rows or (1 << 20)
    v = torch.empty(n, dtype=torch.float32, device=dev)
    gen.device(gen.F32_UNIFORM, v.data_ptr(), n, 0, seed=args.seed, stream=stream.cuda_stream)
    t = float(np.float32(args.selectivity))
    col = [vd.column(v)]
    p = vd.pred([[(0, "<", t)]])
    pos = torch.empty(n, dtype=torch.int32, device=dev)
    cnt = torch.zeros(1, dtype=torch.int64, device=dev)
    ws = vd.alloc_ws(vd.workspace_bytes(vd.VD_OP_SELECT, n), dev)
    flush = torch.empty(512 << 20, dtype=torch.uint8, device=dev)
    res = {}
    launches = 0
    steps = args.steps or 200
    for mode in ("branch", "predicated"):
        sel = vd.select_predicated if mode == "predicated" else vd.select_branch
        plan = plans.selsum(t, vd.VD_SEL_PREDICATED if mode == "predicated" else vd.VD_SEL_BRANCH)
        out = torch.empty(vd.partials_bytes(plan), dtype=torch.uint8, device=dev)
        pws = vd.alloc_ws(vd.workspace_bytes(vd.VD_OP_PIPELINE, n, None, plan), dev)
        calls = {"positions": lambda: sel(col, n, p, out_pos=pos, out_count=cnt, ws=ws, stream=stream),
                 "sum": lambda: vd.run_pipeline(plan, col, n, out=out, ws=pws, stream=stream)}
        for _ in range(max(args.warmup, 3)):
            nl = 0
            for f in calls.values():
                f()
                nl += vd.last_launch_count()
        torch.cuda.synchronize()
        # each call captured once in a CUDA graph and replayed: the events then
        # time the GPU work, not the Python marshalling between launches
        graphs = {}
        side = torch.cuda.Stream(device=dev)
        side.wait_stream(stream)
        for name, f in list(calls.items()) + [("step", lambda: [g() for g in calls.values()])]:
            g = torch.cuda.CUDAGraph()
            with torch.cuda.stream(side):
                with torch.cuda.graph(g, stream=side):
                    if name == "positions":
                        sel(col, n, p, out_pos=pos, out_count=cnt, ws=ws, stream=side)
                    elif name == "sum":
                        vd.run_pipeline(plan, col, n, out=out, ws=pws, stream=side)
                    else:
                        sel(col, n, p, out_pos=pos, out_count=cnt, ws=ws, stream=side)
                        vd.run_pipeline(plan, col, n, out=out, ws=pws, stream=side)
            graphs[name] = g
        stream.wait_stream(side)
        torch.cuda.synchronize()
        r = {}
        for cold in (False, True):
            for name, g in graphs.items():
                f = g.replay
                ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True))
                      for _ in range(steps)]
                for i in range(steps):
                    if cold:
                        flush.fill_(i & 0xFF)  # evict L2 (126 MB) before the call
                    ev[i][0].record(stream)
                    f()
                    ev[i][1].record(stream)
                torch.cuda.synchronize()
                us = sorted(a.elapsed_time(b) * 1e3 for a, b in ev)
                r[f"{name}_{'cold' if cold else 'warm'}_us"] = {"median": statistics.median(us), "best": us[0]}
        launches = max(launches, nl)
        r["launches_per_step"] = nl
        # parity with the oracle (count, positions, f64 sum within 1e-9)
        c = int(cnt.item())
        pos_o, cnt_o, (sh, sl) = oracle.select_f32(v.cpu().numpy(), t, "lt")
        got = vd.decode_partials(out.cpu().numpy().tobytes(), plan, float_aggs=[True])[0]
        r["parity"] = bool(c == cnt_o and np.array_equal(pos[:c].cpu().numpy(), pos_o) and got[1] == cnt_o
                           and abs(got[0] - (sh + sl)) <= 1e-9 * abs(sh + sl))
        r["selected"] = c
        res[mode] = r
    ms = comm.max([res["branch"]["step_warm_us"]["median"] / 1e3])[0]
    line = {"metric": METRIC, "value": n * world / (ms * 1e-3), "unit": "rows/s", "n_gpus": world,
            "steps": steps, "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True,
            "scaling": "weak", "vs_baseline": None, "dtype": "f32/f64", "data": "synthetic (f32 U[0,1), gen/vd_gen.h)",
            "config": bench_config(args, "c1", 0.0, world),
            "c1": res,
            "roofline": {"bound": "latency", "achieved": None, "peak": None, "unit": "us", "frac": None,
                         "traffic": None, "kernel": "k_sel_* + k_pipe_selsum_tma",
                         "note": "4 MiB input + 2 MiB positions are L2-resident: launch/latency-bound by design "
                                 "(SURVEY §8(d) C1); the HBM roofline applies to C2, not here"},
            "clocks": None, "e2e": None, "gpu_launches": launches * steps}
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        cb = cpu_baseline("select", 0.0, args.seed, min(args.cpu_seconds, 5.0), args.selectivity, n)
        if cb is not None:
            line["cpu_baseline"] = cb
    if rank == 0:
        print(json.dumps(line), flush=True)
    comm.close()


class Comm:
    """The cross-rank plumbing of the bench (torch.distributed): NCCL over
    NVLink on device tensors, or gloo on host copies (test mode: several
    ranks may share one GPU)."""

    def __init__(self, world, backend, dev):
        import torch.distributed as dist
        self.world, self.backend, self.dev, self.dist = world, backend, dev, dist
        if world > 1:
            if backend == "nccl":
                dist.init_process_group("nccl", device_id=dev)
            else:
                dist.init_process_group("gloo")

    def barrier(self):
        if self.world > 1:
            self.dist.barrier()

    def all_gather(self, local, gathered):
        if self.world == 1:
            return
        if self.backend == "nccl":
            self.dist.all_gather_into_tensor(gathered, local)
        else:
            h = local.cpu()
            g = gathered.new_empty(gathered.shape, device="cpu")
            self.dist.all_gather_into_tensor(g, h)
            gathered.copy_(g)

    def max(self, vals):
        if self.world == 1:
            return vals
        import torch
        t = torch.tensor(vals, dtype=torch.float64, device=self.dev if self.backend == "nccl" else "cpu")
        self.dist.all_reduce(t, op=self.dist.ReduceOp.MAX)
        return [float(x) for x in t.tolist()]

    def close(self):
        if self.world > 1:
            self.dist.barrier()
            self.dist.destroy_process_group()


def fig14_main(args, rank, world, local):
    """Multi-column FK lookups (Fig 14): n positions resolved
    into the two int32 columns of a target table of --target-mb, by a Single
    Loop (vd_gather_multi), Separate Loops (one vd_gather per column), or a
    Layout Transform (vd_zip of the target into 8-byte rows, inside the timed
    step, then vd_gather_rows).  Lookups are sequential (i mod m) or uniform
    random.  Algorithmic bytes (reading A35, the rule Fig 16 uses, A33): per
    position 4 B read + 2 x 4 B written; a random lookup into a target
    column larger than L2 moves one 64-byte HBM block per column it touches
    (Single / Separate: 2 blocks, Layout: 1 block of the zipped row), plus
    the zip pass's 16 B per target row; sequential lookups and targets that
    fit L2 read the target once (8 B per target row)."""
    import torch

    import gen
    from paper_journals_pvldb_pirkmzm16_b200 import vd

    ndev = torch.cuda.device_count()
    torch.cuda.set_device(local % ndev)
    dev = torch.device("cuda", local % ndev)
    comm = Comm(world, args.dist_backend, dev)
    stream = torch.cuda.current_stream()
    n_total = args.rows or 200_000_000
    a, b = rank * n_total // world, (rank + 1) * n_total // world
    n = b - a
    m = args.target_mb * (1 << 20) // 8
    t0 = torch.empty(m, dtype=torch.int32, device=dev)
    t1 = torch.empty(m, dtype=torch.int32, device=dev)
    gen.device(gen.I32_UNIFORM, t0.data_ptr(), m, 0, seed=args.seed + 3, p0=0, p1=10**9, stream=stream.cuda_stream)
    gen.device(gen.I32_UNIFORM, t1.data_ptr(), m, 0, seed=args.seed + 4, p0=0, p1=10**9, stream=stream.cuda_stream)
    pos = torch.empty(n, dtype=torch.int32, device=dev)
    if args.pattern == "random":
        gen.device(gen.I32_UNIFORM, pos.data_ptr(), n, a, seed=args.seed + 5, p0=0, p1=m - 1, stream=stream.cuda_stream)
    else:
        torch.remainder(torch.arange(a, b, device=dev, dtype=torch.int64), m, out=pos)
    o0 = torch.empty(n, dtype=torch.int32, device=dev)
    o1 = torch.empty(n, dtype=torch.int32, device=dev)
    cols = [vd.column(t0), vd.column(t1)]
    dts = [vd.VD_I32, vd.VD_I32]
    _, stride = vd.row_layout(dts)
    rows = torch.empty(m * stride, dtype=torch.uint8, device=dev)
    launches = {"single": 1, "separate": 2, "layout": 2}[args.strategy]

    def step():
        if args.strategy == "single":
            vd.gather_multi(cols, pos, n, 0, [o0, o1], stream=stream)
        elif args.strategy == "separate":
            vd.gather(cols[0], pos, n, 0, o0, stream=stream)
            vd.gather(cols[1], pos, n, 0, o1, stream=stream)
        else:
            vd.zip_rows(cols, rows, stream=stream)
            vd.gather_rows(rows, m, dts, pos, n, 0, [o0, o1], stream=stream)

    for _ in range(max(args.warmup, 3)):
        step()
    torch.cuda.synchronize()
    ok = bool(torch.equal(o0, t0[pos.long()])) and bool(torch.equal(o1, t1[pos.long()]))
    steps = args.steps or 50
    clocks = ClockSampler(local)
    clocks.start()
    time.sleep(0.3)
    comm.barrier()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(stream)
    for _ in range(steps):
        step()
    e1.record(stream)
    torch.cuda.synchronize()
    clk = clocks.stop()
    ms = comm.max([e0.elapsed_time(e1) / steps])[0]
    col_bytes = m * 4
    big = args.pattern == "random" and col_bytes > 126 * (1 << 20)
    if big:
        look = (64 if args.strategy == "layout" else 128) * n
    else:
        look = 8 * m
    zip_b = 16 * m if args.strategy == "layout" else 0
    alg_bytes = 12 * n + look + zip_b
    alg = alg_bytes / (ms * 1e-3) / 1e9
    line = {"metric": METRIC, "value": n_total / (ms * 1e-3), "unit": "rows/s", "n_gpus": world, "steps": steps,
            "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True, "scaling": "strong",
            "vs_baseline": None, "dtype": "int32", "data": "synthetic (uniform int32 target, gen/vd_gen.h)",
            "config": {"workload": f"fig14_{args.strategy}_{args.pattern}_{args.target_mb}MB_{n_total}",
                       "strategy": args.strategy, "pattern": args.pattern, "target_mb": args.target_mb,
                       "positions": n_total, "target_column_mb": col_bytes / 2**20,
                       "l2": "positions + outputs 2.4 GB per step > 126 MB L2"},
            "roofline": hbm_roofline(alg, {"single": "k_gather", "separate": "k_gather x2",
                                           "layout": "k_zip + k_gather_rows"}[args.strategy], ms, None,
                                     bytes_per_row=alg_bytes / n, lookup_model=(
                                         "64 B HBM block per column lookup (A33/A35)" if big else
                                         "target read once (sequential or L2-resident)")),
            "clocks": clk, "e2e": None, "gpu_launches": launches * steps, "result_ok": ok}
    if rank == 0:
        print(json.dumps(line), flush=True)
    comm.close()


def q19_late_bytes(plan, cols, dims, result, clk, kernel_ms):
    """Algorithmic bytes of the Q19 late-materialisation fragment (A31/A33)."""
    import torch

    import gen
    from paper_journals_pvldb_pirkmzm16_b200 import plans
    mode, instr = cols[4], cols[5]
    codes_m = [i for i, s in enumerate(gen.SHIPMODE) if s in ("AIR", "AIR REG")]
    lead = (instr == gen.SHIPINSTRUCT.index("DELIVER IN PERSON"))
    lead &= torch.isin(mode, torch.tensor(codes_m, dtype=mode.dtype, device=mode.device))
    n = lead.numel()

    def blocks(mask, esz):
        r = 64 // esz
        full = n // r * r
        return 64 * (int(mask[:full].view(-1, r).any(1).sum().item()) + int(bool(mask[full:].any().item())))

    nlead = int(lead.sum().item())
    qual = int(next(iter(result.values()))[-1]) if result else 0
    # k_pipe_late's order: l_partkey, then the equality / IN lookups (p_brand,
    # p_container); l_quantity and p_size only for rows those leave undecided
    # (some branch's brand and container match); the aggregate inputs only
    # for qualifying rows
    idx = lead.nonzero().squeeze(1)
    pk = cols[0][idx].long() - 1
    br, ct = dims[0][pk].long(), dims[1][pk].long()
    und = torch.zeros_like(br, dtype=torch.bool)
    for b, conts, _, _ in plans.Q19_BRANCHES:
        und |= (br == gen.BRAND.index(b)) & torch.isin(ct, torch.tensor([gen.CONTAINER.index(x) for x in conts],
                                                                         device=ct.device))
    iu = idx[und]
    qty, sz = cols[1][iu].long(), dims[2][pk[und]].long()
    ok = torch.zeros_like(qty, dtype=torch.bool)
    for b, conts, qlo, smax in plans.Q19_BRANCHES:
        ok |= ((br[und] == gen.BRAND.index(b))
               & torch.isin(ct[und], torch.tensor([gen.CONTAINER.index(x) for x in conts], device=ct.device))
               & (qty >= qlo * 100) & (qty <= (qlo + 10) * 100) & (sz >= 1) & (sz <= smax))
    und_mask = torch.zeros(n, dtype=torch.bool, device=lead.device)
    und_mask[iu] = True
    full_mask = torch.zeros(n, dtype=torch.bool, device=lead.device)
    full_mask[iu[ok]] = True
    alg = 2 * n + blocks(lead, cols[0].element_size()) + blocks(und_mask, cols[1].element_size())
    alg += blocks(full_mask, cols[2].element_size()) + blocks(full_mask, cols[3].element_size())
    alg += sum(d.numel() * d.element_size() for d in dims)
    clk_ghz = (clk or {}).get("sm_mhz") or 1965.0
    cap = L2_CAP_BYTES_PER_CLK * clk_ghz / 1e3 / 32
    nund = int(und.sum().item())
    sectors = 2 * nlead + nund
    ach = sectors / (kernel_ms * 1e6)
    extra = {"bytes_per_row_dense": BYTES_PER_ROW["q19"], "lead_rows": nlead, "undecided_rows": nund,
             "qualifying_rows": qual, "qualifying_check": int(ok.sum().item()),
             "l2": {"bound": "l2", "lookups": sectors, "achieved_lookups_only": ach, "peak": cap,
                    "unit": "sectors/ns", "frac": ach / cap,
                    "peak_kind": "guide: B300-measured LTS cap 6300 B/clk x SM clock (B300_MICROARCH.md)"}}
    return alg, extra


def q15_main(args, rank, world, local, sf):
    """NEXT-4: TPC-H Q15's revenue view -- shipdate in [1996-01-01,
    1996-04-01), GROUP BY l_suppkey (10,000 x SF groups: a key domain far
    beyond a shared-memory table), SUM(ext * (100 - disc)), COUNT(*) --
    through vd_group_fold (identity hashing over min..max, one streaming pass
    into the global table + the FoldSelect compaction) or, with
    --grouping hash, vd_hash_group_fold (open addressing, shared-memory tables
    spilling to a global one, sized from the distinct-key bound).  N > 1: row
    ranges per rank; every rank's compacted groups go into a fixed-stride
    buffer, one all-gather (counts + groups), then vd_merge_groups (the
    cross-GPU merge of compacted groups, 128-bit sums) -- the step ends with
    the merged groups on every rank.  Algorithmic bytes (A31): the filter
    column in full and, of the other columns, the 64-byte blocks holding a
    qualifying row."""
    import torch

    import gen
    from paper_journals_pvldb_pirkmzm16_b200 import vd

    torch.cuda.set_device(local % torch.cuda.device_count())
    dev = torch.device("cuda", local % torch.cuda.device_count())
    comm = Comm(world, args.dist_backend, dev)
    stream = torch.cuda.current_stream()
    n_total = gen.lineitem_rows(sf)
    a0, b0 = rank * n_total // world, (rank + 1) * n_total // world
    n = b0 - a0
    names = ["l_shipdate", "l_suppkey", "l_extendedprice", "l_discount"]
    cols = []
    for nm in names:
        col = gen.LINEITEM_COLS[nm]
        t = torch.empty(n, dtype=getattr(torch, _dt(col)), device=dev)
        gen.device(col, t.data_ptr(), n, a0, sf=sf, seed=args.seed, stream=stream.cuda_stream)
        cols.append(t)
    torch.cuda.synchronize()
    views = [vd.describe(t, stream=stream) for t in cols]
    # every rank sizes its table from the key column's global domain (the
    # supplier table's key range: 1 .. 10000 x SF), so strides agree
    kmin, kmax = 1, gen.supplier_rows(sf)
    views[1].min, views[1].max, views[1].has_minmax = kmin, kmax, 1
    p = vd.pred([[(0, ">=", 9496), (0, "<", 9587)]])
    aggs = [("sum", [2, (3, 100, -1)]), ("count",)]
    D = kmax - kmin + 1
    hashed = args.grouping == "hash"
    keys = torch.empty(D, dtype=torch.int64, device=dev)
    rows = torch.empty(D, dtype=torch.int64, device=dev)
    slots = torch.empty(D * len(aggs) * 16, dtype=torch.uint8, device=dev)
    ng = torch.zeros(1, dtype=torch.int64, device=dev)
    if hashed:
        ws = vd.alloc_ws(vd.hash_group_fold_ws_bytes(D, len(aggs)), dev)
    else:
        ws = vd.alloc_ws(vd.group_fold_ws_bytes(D, len(aggs)), dev)
    if world > 1:
        gk = torch.empty(D * world, dtype=torch.int64, device=dev)
        gr = torch.empty(D * world, dtype=torch.int64, device=dev)
        gs = torch.empty(D * world * len(aggs) * 16, dtype=torch.uint8, device=dev)
        gn = torch.empty(world, dtype=torch.int64, device=dev)
        mk = torch.empty(D, dtype=torch.int64, device=dev)
        mr = torch.empty(D, dtype=torch.int64, device=dev)
        ms_ = torch.empty(D * len(aggs) * 16, dtype=torch.uint8, device=dev)
        mn = torch.empty(1, dtype=torch.int64, device=dev)
        mws = vd.alloc_ws(vd.merge_groups_ws_bytes(D, len(aggs)), dev)

    def step():
        if hashed:
            vd.hash_group_fold(views, n, 1, aggs, p, max_groups=D, out_keys=keys, out_aggs=slots, out_rows=rows,
                               out_ngroups=ng, ws=ws, stream=stream)
        else:
            vd.group_fold(views, n, 1, aggs, p, out_keys=keys, out_aggs=slots, out_rows=rows, out_ngroups=ng,
                          ws=ws, stream=stream)
        if world > 1:
            comm.all_gather(ng, gn)
            comm.all_gather(keys, gk)
            comm.all_gather(rows, gr)
            comm.all_gather(slots, gs)
            vd.merge_groups(gk, gs, gr, gn, world, D, [vd.VD_AGG_SUM, vd.VD_AGG_COUNT], [False, False],
                            max_groups=D, out_keys=mk, out_aggs=ms_, out_rows=mr, out_ngroups=mn, ws=mws,
                            stream=stream)

    for _ in range(max(args.warmup, 3)):
        step()
    launches = vd.last_launch_count()
    torch.cuda.synchronize()
    steps = args.steps or 50
    clocks = ClockSampler(local)
    clocks.start()
    time.sleep(0.3)
    comm.barrier()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(stream)
    for _ in range(steps):
        step()
    e1.record(stream)
    torch.cuda.synchronize()
    comm.barrier()
    clk = clocks.stop()
    ms = comm.max([e0.elapsed_time(e1) / steps])[0]
    rk, rr, rs, rn = (mk, mr, ms_, mn) if world > 1 else (keys, rows, slots, ng)
    g = int(rn.item())
    order = torch.argsort(rk[:g])  # a canonical order for the digest (hash output is in table order)
    kk = rk[:g][order].cpu().numpy()
    rowsv = rr[:g][order].cpu().numpy()
    sl = rs[:g * 32].view(g, 32)[order].cpu().numpy()
    digest = __import__("hashlib").sha256(kk.tobytes() + rowsv.tobytes() + sl.tobytes()).hexdigest()[:16]
    mask = (cols[0] >= 9496) & (cols[0] < 9587)
    alg_bytes = 4 * n
    for t in cols[1:]:
        r = 64 // t.element_size()
        m = mask[:n // r * r].view(-1, r).any(1)
        alg_bytes += 64 * (int(m.sum().item()) + int(bool(mask[n // r * r:].any().item())))
    sel = float(mask.float().mean().item())
    del mask
    alg = alg_bytes / (ms * 1e-3) / 1e9
    line = {"metric": METRIC, "value": n_total / (ms * 1e-3), "unit": "rows/s", "n_gpus": world, "steps": steps,
            "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True, "scaling": "strong",
            "vs_baseline": None, "dtype": "int64",
            "data": "synthetic (dbgen-shaped, counter-based generator gen/vd_gen.h, generated in HBM)",
            "config": {**bench_config(args, "q15", sf, world), "grouping": args.grouping}, "groups_domain": D,
            "groups": g,
            "roofline": hbm_roofline(alg, ("vd_hash_group_fold" if hashed else "vd_group_fold") +
                                     (" + all-gather + vd_merge_groups" if world > 1 else ""), ms,
                                     ncu_traffic("q15", world), bytes_per_row=alg_bytes / n, dense_bytes_per_row=24,
                                     selectivity=sel),
            "clocks": clk, "e2e": None, "gpu_launches": launches * steps, "result_digest": digest}
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        cb = cpu_baseline("q15", sf, args.seed, args.cpu_seconds, args.selectivity, n)
        if cb is not None:
            line["cpu_baseline"] = cb
    if rank == 0:
        print(json.dumps(line), flush=True)
    comm.close()


def _dt(col):
    import gen
    import numpy as np
    return {np.uint8: "uint8", np.int32: "int32", np.int64: "int64", np.float32: "float32",
            np.float64: "float64"}[gen.dtype_of(col)]


def e2e_measure(args, torch, vd, plan, cols, views, dims, dim_views, n, dev, stream, world, comm, pbytes):
    """Through the public API from pinned host buffers: vd_load_column (H2D)
    of every input column, vd_run_pipeline, D2H of the partials."""
    try:
        host = [torch.empty(c.numel(), dtype=c.dtype, pin_memory=True) for c in cols]
        pinned = True
    except Exception:
        host = [torch.empty(c.numel(), dtype=c.dtype) for c in cols]
        pinned = False
    for h, c in zip(host, cols):
        h.copy_(c)
    dst = [torch.empty_like(c) for c in cols]
    out = torch.empty(pbytes, dtype=torch.uint8, device=dev)
    gathered = torch.empty(pbytes * world, dtype=torch.uint8, device=dev) if world > 1 else out
    result = vd.DeviceResult(plan, dev)
    rbufs = [result.ngroups, result.keys, result.rows, result.aggs]
    hres = [torch.empty(t.numel(), dtype=t.dtype, pin_memory=pinned) for t in rbufs]
    ws = vd.alloc_ws(vd.workspace_bytes(vd.VD_OP_PIPELINE, n, None, plan), dev)
    reps = 3
    torch.cuda.synchronize()
    comm.barrier()
    t0 = time.perf_counter()
    for _ in range(reps):
        vcols = []
        for h, d, v in zip(host, dst, views):
            c = vd.load_column(h, d, compute_minmax=False, stream=stream)
            c.min, c.max, c.has_minmax, c.flags = v.min, v.max, v.has_minmax, v.flags  # catalog metadata
            vcols.append(c)
        vd.run_pipeline(plan, vcols, n, dim_views, out=out, ws=ws, stream=stream)
        comm.all_gather(out, gathered)
        vd.merge_partials_device(plan, vcols, dim_views, gathered, world, result, stream=stream)
        for h, d in zip(hres, rbufs):  # the compacted result back to the host
            h.copy_(d, non_blocking=True)
        torch.cuda.synchronize()
    dt = (time.perf_counter() - t0) / reps
    dt = comm.max([dt])[0]
    h2d = sum(c.numel() * c.element_size() for c in cols)
    d2h = sum(t.numel() * t.element_size() for t in rbufs)
    del host, dst
    return {"value": (n * world) / dt, "unit": "rows/s", "h2d_bytes_per_step": h2d, "d2h_bytes_per_step": d2h,
            "pinned": pinned, "reps": reps, "s_per_step": dt}


def workload_rows(args, w, sf):
    import gen
    if w in ("select", "selpos", "selagg"):
        return args.rows or 10**9
    if w in ("fkjsel", "fig14"):
        return args.rows or 200_000_000
    if w == "c1":
        return args.rows or (1 << 20)
    return gen.lineitem_rows(sf)


def bench_config(args, w, sf, world):
    """The workload's `config` (identical in the GPU arm and the reference
    arm: the driver compares them)."""
    n_total = workload_rows(args, w, sf)
    bpr = BYTES_PER_ROW.get(w, 4)
    name = {"q1": f"tpch_q1_sf{sf:g}", "q6": f"tpch_q6_sf{sf:g}", "q19": f"fkj_q19_sf{sf:g}",
            "q9": f"fkj_q9_sf{sf:g}", "q15": f"tpch_q15_revenue_sf{sf:g}",
            "select": f"select_f32_{n_total}_s{args.selectivity:g}",
            "selagg": f"selagg_f32x2_{n_total}_s{args.selectivity:g}",
            "selpos": f"selpos_f32_{n_total}_s{args.selectivity:g}",
            "c1": f"c1_select_f32_{n_total}_s{args.selectivity:g}",
            "fkjsel": f"fkjsel_{n_total}x{128 * 1024 * 1024}_s{args.selectivity:g}"}.get(w, w)
    per_gpu = n_total // world
    return {"workload": name, "rows": n_total, "rows_per_gpu": per_gpu, "sf": sf, "sel_mode": args.sel_mode,
            **({"materialize": args.materialize, "chunk": args.chunk} if args.materialize != "none" else {}),
            "parallelism": f"row-range x{world}" + (" + NCCL all_gather of partials" if world > 1 else ""),
            "l2": ("inputs L2-resident by design (C1): warm and cold (after a 512 MB L2 flush) reported"
                   if w == "c1" else f"inputs {per_gpu * bpr / 1e9:.1f} GB per GPU > 126 MB L2: no flush needed"),
            "seed": args.seed}


def reference_arm(args, rank, world, sf):
    """The tier's reference arm: the CPU oracle on the same config/metric."""
    if rank != 0:
        return
    w = args.workload
    steps = args.steps if args.steps is not None else 3
    budget = max(1.0, min(args.cpu_seconds, 60.0) / max(steps, 1))
    vals = []
    cb = None
    n_total = workload_rows(args, w, sf)
    if args.warmup > 0:
        cpu_baseline(w, sf, args.seed, 0.5, args.selectivity, n_total, partitioned=False)
    t0 = time.perf_counter()
    for _ in range(steps):
        cb = cpu_baseline(w, sf, args.seed, budget, args.selectivity, n_total, partitioned=False)
        vals.append(cb["value"])
    wall = time.perf_counter() - t0
    v = statistics.median(vals)
    line = {"metric": METRIC, "value": v, "unit": "rows/s", "impl": "reference", "n_gpus": world, "steps": steps,
            "warmup": args.warmup, "ms_per_step": wall / steps * 1e3, "higher_is_better": True, "scaling": "strong",
            "vs_baseline": None, "dtype": "f32/f64" if w in ("select", "selpos", "c1") else "int64",
            "data": "synthetic (dbgen-shaped, counter-based generator gen/vd_gen.h, host)",
            "config": bench_config(args, w, sf, world),
            "cpu_baseline": {"value": v, "unit": "rows/s", "cores": 1, "kind": "oracle", "sample": cb["sample"],
                             **host_info()},
            "e2e": {"value": v, "unit": "rows/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


if __name__ == "__main__":
    main()
