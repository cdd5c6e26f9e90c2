"""Epsilon (the empty slot, §2.1) through the DEFAULT Q1 / Q6 /
selective-sum fragments, and the int64 overflow proofs at the launch shape
that actually runs.

The fused fragments that serve BASELINE.json's headline configs
(``q1_tma``, ``q1_ldg``, ``scalar_tma``, ``selsum_tma``) must honour vd.h's epsilon contract
exactly like the generic fragment: a term over epsilon is false (A9), an
epsilon group-key code gives the row no group (Partition drops it), and an
epsilon factor makes that aggregate's value epsilon -- skipped by the SUM
(A5) while the row still counts (COUNT(*)).  Expected values come from the
oracle's literal interpreter running programs.Q1 / programs.Q6 with the
same epsilon masks (the Fig 10/11 and Fig 8 plan shapes).
"""
import numpy as np
import pytest
import torch

import gen
import oracle
from oracle import programs
from paper_journals_pvldb_pirkmzm16_b200 import plans, vd

from test_gpu_pipeline import env, lineitem, load, run

pytestmark = pytest.mark.gpu

EPS_OF = {np.dtype(np.uint8): 0xFF, np.dtype(np.int32): -2**31, np.dtype(np.int64): -2**63}


def inject_eps(cols, names, frac, seed):
    """Epsilon sentinels in a fraction of every named column; returns the masks."""
    rng = np.random.default_rng(seed)
    masks = {}
    for c in names:
        m = rng.random(len(cols[c])) < frac
        cols[c] = cols[c].copy()
        cols[c][m] = EPS_OF[cols[c].dtype]
        masks[c] = m
    return masks


# COUNT(*) per group = FoldCount over the (never-epsilon once scattered)
# group key; the groups kept are those with at least one row.
Q1_ROWS = """
rows := FoldCount(sc.key, sc.key)
gpos2 := FoldSelect(rows)
r_key := Gather(gkey, gpos2)
r_qty := Gather(s_qty, gpos2)
r_base := Gather(s_base, gpos2)
r_dp := Gather(s_dp, gpos2)
r_ch := Gather(s_ch, gpos2)
r_disc := Gather(s_disc, gpos2)
r_rows := Gather(rows, gpos2)
"""


def q1_interpreter(li, masks):
    p = oracle.Program()
    for c in plans.Q1_COLS:
        p.set("lineitem." + c, li[c], masks.get(c))
    p.run(programs.Q1.format(ship_max_p1=plans.Q1_SHIP_MAX + 1) + Q1_ROWS)
    keys = p.get("r_key")
    outs = [p.get(o) for o in ("r_qty", "r_base", "r_dp", "r_ch", "r_disc", "r_rows")]
    # FoldSelect output (and so every Gather through it) is epsilon-padded
    # past the selected groups (Fig 11)
    return {k: [(o[j] or 0) for o in outs] for j, k in enumerate(keys) if k is not None}


@pytest.mark.parametrize("variant", ["q1_tma", "q1_ldg"])
@pytest.mark.parametrize("sel_mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED])
@pytest.mark.parametrize("n", [5003, 262147])
def test_q1_epsilon_vs_interpreter(variant, sel_mode, n):
    li = lineitem(0.1, n)
    masks = inject_eps(li, plans.Q1_COLS, 0.02, seed=n + 17)
    exp = q1_interpreter(li, masks)
    keep, views = load([li[c] for c in plans.Q1_COLS])
    assert all(not (v.flags & vd.VD_COL_NOEPS) for v in views)
    plan = plans.q1(sel_mode)
    with env(VD_Q1_VARIANT="ldg" if variant == "q1_ldg" else "tma"):
        buf, nl = run(plan, views, n, want=(variant,))
    got = vd.decode_partials(buf, plan)
    assert {k: v[:5] + [v[6]] for k, v in got.items()} == exp
    for v in got.values():
        assert v[5] == v[6]  # COUNT(*) aggregate == row count
    # the generic fragment agrees on the same epsilon-laden input
    gbuf, _ = run(plans.q1(sel_mode, force_generic=True), views, n, want=("generic",))
    assert gbuf == buf


def test_q1_epsilon_only_in_ship_date_one_sided_filter():
    """`l_shipdate <= c` is one-sided: the planner's interval must still
    exclude INT32_MIN (epsilon), else every epsilon ship date qualifies."""
    n = 70001
    li = lineitem(0.1, n)
    masks = inject_eps(li, ["l_shipdate"], 0.3, seed=5)
    exp = q1_interpreter(li, masks)
    keep, views = load([li[c] for c in plans.Q1_COLS])
    got = vd.decode_partials(run(plans.q1(), views, n, want=("q1_tma",))[0], plans.q1())
    assert {k: v[:5] + [v[6]] for k, v in got.items()} == exp


def test_q1_epsilon_keys_never_index_outside_the_table():
    """An epsilon u8 key (0xFF) must not address the shared-memory group
    table: every row's keys are epsilon except a few."""
    n = 40000
    li = lineitem(0.1, n)
    masks = inject_eps(li, ["l_returnflag"], 0.97, seed=9)
    exp = q1_interpreter(li, masks)
    keep, views = load([li[c] for c in plans.Q1_COLS])
    got = vd.decode_partials(run(plans.q1(), views, n, want=("q1_tma",))[0], plans.q1())
    assert {k: v[:5] + [v[6]] for k, v in got.items()} == exp


Q6_COUNT = """
pc2 := FoldCount(fold, positions)
count2 := FoldSum(pc2)
"""


def q6_interpreter(li, masks):
    p = oracle.Program()
    for c in plans.Q6_COLS:
        p.set("lineitem." + c, li[c], masks.get(c))
    p.run(programs.Q6.format(intent=4096, d0m1=8765, d1=9131, dlom1=4, dhip1=8, qmax=2400) + Q6_COUNT)
    return (p.get("revenue")[0] or 0), p.get("count2")[0]


@pytest.mark.parametrize("variant", ["tma", "ldg"])
@pytest.mark.parametrize("sel_mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED])
@pytest.mark.parametrize("n", [4097, 300007])
def test_q6_epsilon_vs_interpreter(variant, sel_mode, n):
    li = lineitem(0.1, n)
    # a wider window than Q6's so that many rows qualify
    masks = inject_eps(li, plans.Q6_COLS, 0.03, seed=n + 3)
    exp = q6_interpreter(li, masks)
    keep, views = load([li[c] for c in plans.Q6_COLS])
    plan = plans.q6(sel_mode)
    with env(VD_SCALAR_VARIANT=variant):
        buf, _ = run(plan, views, n, want=("scalar_" + variant,))
    got = vd.decode_partials(buf, plan)[0]
    assert (got[0], got[2]) == exp
    assert got[1] == got[2]
    gbuf, _ = run(plans.q6(sel_mode, force_generic=True), views, n, want=("generic",))
    assert gbuf == buf


def test_q6_epsilon_only_in_quantity_one_sided_filter():
    """`l_quantity < 2400` is one-sided: epsilon (INT64_MIN) must not pass."""
    n = 200003
    li = lineitem(0.1, n)
    masks = inject_eps(li, ["l_quantity"], 0.5, seed=21)
    exp = q6_interpreter(li, masks)
    keep, views = load([li[c] for c in plans.Q6_COLS])
    got = vd.decode_partials(run(plans.q6(), views, n, want=("scalar_tma",))[0], plans.q6())[0]
    assert (got[0], got[2]) == exp


SELSUM2 = """
v := Load(input)
keep := Greater({t}, v.x)
positions := FoldSelect(keep)
sel := Gather(v.y, positions)
total := FoldSum(sel)
count := FoldCount(positions)
"""


@pytest.mark.parametrize("sel_mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED])
def test_f32_selective_sum_of_another_column_with_nan(sel_mode):
    """Selective sum of column y over a filter on column x (both f32), NaN
    (epsilon) in both: NaN never passes the filter, a NaN value is skipped
    by the FoldSum while its row counts.  f64 accumulation, rel 1e-9."""
    n = 3 * 8192 * 5 + 77
    x = gen.host(gen.F32_UNIFORM, n, seed=1)
    y = gen.host(gen.F32_UNIFORM, n, seed=2)
    rng = np.random.default_rng(4)
    mx, my = rng.random(n) < 0.05, rng.random(n) < 0.05
    x[mx] = np.nan
    y[my] = np.nan
    t = float(np.float32(0.6))
    p = oracle.Program()
    p.set("input.x", np.where(mx, 0, x), mx)
    p.set("input.y", np.where(my, 0, y), my)
    p.run(SELSUM2.format(t=repr(t)))
    v, r, _ = p.get_float_exact("total")
    exp_sum, exp_cnt = v[0] + r[0], p.get("count")[0]
    dx, dy = torch.from_numpy(x).cuda(), torch.from_numpy(y).cuda()
    plan = vd.pipeline(pred_=vd.pred([[(0, "<", t)]]), sel_mode=sel_mode, aggs=[("sum", [1]), ("count",)])
    buf, _ = run(plan, [vd.column(dx), vd.column(dy)], n, want=("selsum_tma",))
    # the per-row scalar fragment (VD_SCALAR_VARIANT=ldg) agrees
    with env(VD_SCALAR_VARIANT="ldg"):
        lbuf, _ = run(plan, [vd.column(dx), vd.column(dy)], n, want=("scalar_ldg",))
    lgot = vd.decode_partials(lbuf, plan, float_aggs=[True])[0]
    assert lgot[1] == exp_cnt and abs(lgot[0] - exp_sum) <= 1e-9 * abs(exp_sum)
    got = vd.decode_partials(buf, plan, float_aggs=[True])[0]
    assert got[1] == exp_cnt and got[2] == exp_cnt
    assert abs(got[0] - exp_sum) <= 1e-9 * abs(exp_sum)


# ---- overflow proofs at the launch shape that runs ----------------------------------
def _sms():
    return torch.cuda.get_device_properties(0).multi_processor_count


def _q1_table(n, ext):
    """Every row qualifies and lands in one group with the largest charge
    factor (disc 0, tax 8): per-warp int64 sums are as large as the data allows."""
    li = {"l_shipdate": np.full(n, 9000, np.int32), "l_returnflag": np.zeros(n, np.uint8),
          "l_linestatus": np.zeros(n, np.uint8), "l_quantity": np.full(n, 100, np.int64),
          "l_extendedprice": np.full(n, ext, np.int64), "l_discount": np.zeros(n, np.int64),
          "l_tax": np.full(n, 8, np.int64)}
    li["l_discount"][::7] = 10
    li["l_tax"][::5] = 0
    return li


def test_q1_overflow_bound_uses_the_tma_launch_shape():
    """The Q1 TMA launch has sms CTAs x 8 consumer warps; a warp folds 128
    rows of each of its CTA's tiles (+ <= 128 tail rows on CTA 0) into int64
    slots.  Data just under that bound runs q1_tma exactly; data over it --
    but under the bound the planner used to compute for a 2x wider grid --
    must take the 128-bit generic path, and does overflow int64 per warp."""
    sms = _sms()
    n = 1024 * sms * 8 + 333
    rpw = -(-(n // 1024) // sms) * 128 + 128
    old_rpw = -(-n // (2 * sms * 256)) * 32 + 64
    ok_ext = int(9.0e18 / rpw / 10800.0 * 0.97)
    over_ext = int(9.0e18 / old_rpw / 10800.0 * 0.95)  # the old proof accepted this
    assert over_ext * 10800.0 * rpw > 9.0e18
    for ext, want in ((ok_ext, "q1_tma"), (over_ext, "generic")):
        li = _q1_table(n, ext)
        exp = oracle.q1(li)
        keep, views = load([li[c] for c in plans.Q1_COLS])
        buf, _ = run(plans.q1(), views, n, want=(want,))
        got = vd.decode_partials(buf, plans.q1())
        assert {k: v[:6] for k, v in got.items()} == exp
        # exact charge sum of warp 0 of CTA 0 (tiles 0, sms, 2 sms, ...)
        rows = np.concatenate([np.arange(t * 1024, t * 1024 + 128) for t in range(0, n // 1024, sms)])
        ch = sum(int(li["l_extendedprice"][r]) * (100 - int(li["l_discount"][r])) * (100 + int(li["l_tax"][r]))
                 for r in rows)
        assert (ch < 2**63) == (want == "q1_tma")


def test_q6_overflow_bound_uses_the_scalar_launch_shape():
    """The Q6 TMA launch has sms CTAs x 256 consumer threads; a thread folds
    8 rows of each of its CTA's 2048-row tiles (+ the tail on CTA 0) into
    one int64 sum.  Same two cases as the Q1 test."""
    sms = _sms()
    n = 2048 * sms * 8 + 1000
    rpt = -(-(n // 2048) // sms) * 8 + 8
    old_rows = -(-n // (4 * sms * 256)) + 8
    ok_ext = int(9.0e18 / rpt / 7.0 * 0.97)
    over_ext = int(9.0e18 / old_rows / 7.0 * 0.95)
    assert over_ext * 7.0 * rpt > 9.0e18
    for ext, want in ((ok_ext, "scalar_tma"), (over_ext, "generic")):
        li = {"l_shipdate": np.full(n, 9000, np.int32), "l_discount": np.full(n, 7, np.int64),
              "l_quantity": np.full(n, 100, np.int64), "l_extendedprice": np.full(n, ext, np.int64)}
        li["l_discount"][::3] = 5
        rev, cnt = oracle.q6(li)
        keep, views = load([li[c] for c in plans.Q6_COLS])
        got = vd.decode_partials(run(plans.q6(), views, n, want=(want,))[0], plans.q6())[0]
        assert (got[0], got[2]) == (rev, cnt)
        # exact sum of thread 0 of CTA 0: rows t*2048 + 256 k of its tiles
        rows = np.concatenate([np.arange(t * 2048, t * 2048 + 2048, 256) for t in range(0, n // 2048, sms)])
        s = sum(int(li["l_extendedprice"][r]) * int(li["l_discount"][r]) for r in rows)
        assert (s < 2**63) == (want == "scalar_tma")
