"""vd_merge_partials_device: the cross-GPU step of the hierarchical fold
(Fig 3 one level up) plus the Fig 11 compaction
on the device, against the oracle.

The partials of G "ranks" are produced by the library itself from row-range
shards of one table (vd_run_pipeline on each shard: the launch configuration
bench.py times), gathered back to back as an all-gather would leave them,
merged + compacted on the device, and compared with the oracle's result on
the WHOLE table (pin P8: shards merge to the whole).  Synthetic partials
cover what real shards rarely do: groups empty on some ranks, MIN/MAX, f64
sums, 128-bit carries, and more groups than the kernel's 256-group chunk.
"""
import struct

import numpy as np
import pytest
import torch

import gen
import oracle
from paper_journals_pvldb_pirkmzm16_b200 import plans, vd

from test_gpu_pipeline import lineitem, load

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("G", [1, 2, 3, 8])
def test_q1_shards_merged_on_device_equal_whole_table(G):
    n = 300007
    li = lineitem(0.1, n)
    exp = oracle.q1(li)
    keep, views = load([li[c] for c in plans.Q1_COLS])
    plan = plans.q1()
    nb = vd.partials_bytes(plan)
    gathered = torch.empty(nb * G, dtype=torch.uint8, device="cuda")
    for r in range(G):
        a, b = r * n // G, (r + 1) * n // G
        sv = []
        for v, t in zip(views, keep):
            c = vd.column(t[a:b], minmax=(v.min, v.max), noeps=bool(v.flags & vd.VD_COL_NOEPS))
            sv.append(c)
        vd.run_pipeline(plan, sv, b - a, out=gathered[r * nb:(r + 1) * nb])
    res = vd.merge_partials_device(plan, views, [], gathered, G)
    got = res.decode(plan)
    assert {k: v[:6] for k, v in got.items()} == exp
    assert list(got) == sorted(exp)  # ascending key (A16)
    assert vd.last_launch_count() == 1


def _pack(vals):
    b = b""
    for v in vals:
        if isinstance(v, float):
            b += struct.pack("<dq", v, 0)
        else:
            b += struct.pack("<Qq", v & (2**64 - 1), v >> 64)
    return b


@pytest.mark.parametrize("ngroups,nparts", [(1, 1), (7, 3), (600, 5), (4096, 8)])
def test_device_merge_equals_host_merge_synthetic(ngroups, nparts):
    """Random partials (some groups empty on some or all ranks; int128
    sums near 2^100; f64 sums; integer MIN/MAX) merged on the device equal
    the library's host merge, which the CPU tests pin (test_abi)."""
    rng = np.random.default_rng(ngroups * 31 + nparts)
    plan = vd.pipeline(key=[(0, 0, 0, 1)], ngroups=ngroups,
                       aggs=[("sum", [1]), ("sum", [2]), ("min", [1]), ("max", [1]), ("count",)])
    c0, c1, c2 = vd.column_meta(vd.VD_I32), vd.column_meta(vd.VD_I64), vd.column_meta(vd.VD_F64)
    parts = []
    for r in range(nparts):
        vals = []
        for g in range(ngroups):
            rows = int(rng.integers(1, 1000)) if rng.random() < 0.6 else 0
            if rows:
                big = int(rng.integers(-2**62, 2**62)) * 2**38 + int(rng.integers(0, 2**38))  # ~2^100
                vals += [big, float(rng.random() * 1e6),
                         int(rng.integers(-2**62, 2**62)), int(rng.integers(-2**62, 2**62)), rows, rows]
            else:
                vals += [0, 0.0, 0, 0, 0, 0]
        parts.append(_pack(vals))
    fl = [False, True]
    host = vd.merge_partials(plan, [c0, c1, c2], [], parts, float_aggs=fl)
    dev = torch.from_numpy(np.frombuffer(b"".join(parts), dtype=np.uint8).copy()).cuda()
    got = vd.merge_partials_device(plan, [c0, c1, c2], [], dev, nparts).decode(plan, float_aggs=fl)
    assert got == host
    assert list(got) == sorted(got)


def test_device_merge_rejects_small_capacity():
    plan = plans.q1()
    res = vd.DeviceResult(plan)
    res.struct.capacity = 3
    with pytest.raises(vd.VdError):
        vd.merge_partials_device(plan, [], [], torch.zeros(vd.partials_bytes(plan), dtype=torch.uint8,
                                                           device="cuda"), 1, res)
