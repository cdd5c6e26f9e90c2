"""Materialising plans of vd_run_pipeline against the
oracle: Break (the predicate materialised, Fig 8) and Materialize
(per-chunk position lists, the Vectorized plan of Fig 15),
each followed by a second loop that resolves the rows and folds.

- Fig 15's selective aggregation (sum of v2 where v1 between lo and hi, f32
  with f64 accumulation): against the interpreter running FIG15_VECTORIZED /
  FIG15_BREAK (the programs with the Materialize / Break operator), count
  exact, sum within 1e-9 relative (north_star).
- Integer plans (Q6 scalar, Q1 grouped, the Q19 / Q9 FK joins): bit-exact
  against the brute-force oracle, every chunk size class (32 rows, the
  1024 default, chunks longer than the table), ragged tails.
"""
import numpy as np
import pytest
import torch

import gen
import oracle
from oracle import programs
from paper_journals_pvldb_pirkmzm16_b200 import plans, vd

from test_gpu_pipeline import _dims, lineitem, load, run

pytestmark = pytest.mark.gpu

MATS = [(vd.VD_MAT_BREAK, 0), (vd.VD_MAT_CHUNKS, 32), (vd.VD_MAT_CHUNKS, 0), (vd.VD_MAT_CHUNKS, 1 << 20)]
FRAG = {vd.VD_MAT_BREAK: "break", vd.VD_MAT_CHUNKS: "mat_chunks"}


@pytest.mark.parametrize("mat,chunk", MATS)
@pytest.mark.parametrize("sel_mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED])
@pytest.mark.parametrize("n", [7, 70001, 1 << 20])
def test_fig15_selagg_materialised_vs_interpreter(mat, chunk, sel_mode, n):
    v1 = gen.host(gen.F32_UNIFORM, n, seed=21)
    v2 = gen.host(gen.F32_UNIFORM, n, seed=22)
    v1[::17] = np.nan  # epsilon never qualifies (A9)
    m1 = np.isnan(v1)
    lo, hi = np.float32(0.2), np.float32(0.7)
    lom = float(np.nextafter(lo, np.float32(-1)))
    hip = float(np.nextafter(hi, np.float32(2)))
    prog = programs.FIG15_BREAK if mat == vd.VD_MAT_BREAK else programs.FIG15_VECTORIZED
    p = oracle.run(prog.format(lom=lom.hex(), hip=hip.hex(), chunk=chunk or 1024),
                   input__v1=(np.where(m1, 0, v1), m1), input__v2=v2)
    t, r, _ = p.get_float_exact("total")
    exp_sum, exp_cnt = t[0] + r[0], p.get("count")[0]
    d1, d2 = torch.from_numpy(v1).cuda(), torch.from_numpy(v2).cuda()
    plan = plans.selagg(float(lo), float(hi), sel_mode, materialize=mat, mat_chunk=chunk)
    buf, nl = run(plan, [vd.column(d1), vd.column(d2)], n, want=(FRAG[mat],))
    got = vd.decode_partials(buf, plan, float_aggs=[True])[0]
    assert got[1] == exp_cnt and got[2] == exp_cnt
    assert abs(got[0] - exp_sum) <= 1e-9 * abs(exp_sum)
    assert nl == 2  # the breaker's loop + the folding loop
    # the fused plan on the same input agrees
    fbuf, fnl = run(plans.selagg(float(lo), float(hi), sel_mode), [vd.column(d1), vd.column(d2)], n,
                    want=("selsum_tma",))
    fused = vd.decode_partials(fbuf, plan, float_aggs=[True])[0]
    assert fused[1] == exp_cnt and abs(fused[0] - exp_sum) <= 1e-9 * abs(exp_sum) and fnl == 1


@pytest.mark.parametrize("mat,chunk", MATS)
@pytest.mark.parametrize("n", [4097, 600011])
def test_q6_materialised_exact(mat, chunk, n):
    li = lineitem(0.1, n)
    exp = oracle.q6(li)
    keep, views = load([li[c] for c in plans.Q6_COLS])
    plan = plans.q6()
    plan.materialize, plan.mat_chunk = mat, chunk
    got = vd.decode_partials(run(plan, views, n, want=(FRAG[mat],))[0], plan)[0]
    assert (got[0], got[2]) == exp and got[1] == got[2]


@pytest.mark.parametrize("mat,chunk", MATS)
def test_q1_grouped_materialised_exact(mat, chunk):
    n = 300007
    li = lineitem(0.1, n)
    exp = oracle.q1(li)
    keep, views = load([li[c] for c in plans.Q1_COLS])
    plan = plans.q1()
    plan.materialize, plan.mat_chunk = mat, chunk
    got = vd.decode_partials(run(plan, views, n, want=(FRAG[mat],))[0], plan)
    assert {k: v[:6] for k, v in got.items()} == exp


@pytest.mark.parametrize("variant", [0, 1])
@pytest.mark.parametrize("mat,chunk", [(vd.VD_MAT_BREAK, 0), (vd.VD_MAT_CHUNKS, 0)])
def test_fk_joins_materialised_exact(variant, mat, chunk):
    """Q19-style (predicate over gathered part columns) and Q9-style (no
    predicate, grouped by gathered nation x year): the first loop resolves
    the gathers of the predicate, the second those of the key / values."""
    sf = 0.05
    n = 100003
    li = lineitem(sf, n)
    part, supp = _dims(sf)
    exp = oracle.fkj(variant, li, part, supp)
    codes = {"brand": {b: i for i, b in enumerate(gen.BRAND)},
             "container": {b: i for i, b in enumerate(gen.CONTAINER)},
             "shipmode": {b: i for i, b in enumerate(gen.SHIPMODE)},
             "shipinstruct": {b: i for i, b in enumerate(gen.SHIPINSTRUCT)}}
    if variant == 0:
        plan, names, dn, dt = plans.q19(codes), plans.Q19_COLS, plans.Q19_DIMS, part
    else:
        plan, names, dn, dt = plans.q9(), plans.Q9_COLS, plans.Q9_DIMS, supp
    plan.materialize, plan.mat_chunk = mat, chunk
    keep, views = load([li[c] for c in names])
    dkeep, dviews = load([dt[c] for c in dn])
    got = vd.decode_partials(run(plan, views, n, dviews, want=(FRAG[mat],))[0], plan)
    assert {k: tuple(v[:2]) for k, v in got.items()} == exp


def test_materialise_rejects_bad_chunk():
    n = 1000
    d = torch.zeros(n, dtype=torch.float32, device="cuda")
    plan = plans.selagg(0.1, 0.2, materialize=vd.VD_MAT_CHUNKS, mat_chunk=100)
    out = torch.empty(vd.partials_bytes(plan), dtype=torch.uint8, device="cuda")
    with pytest.raises(vd.VdError):
        vd.run_pipeline(plan, [vd.column(d), vd.column(d)], n, out=out)
