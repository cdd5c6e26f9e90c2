"""GPU parity of vd_group_fold (grouped fold over a
large key domain, identity hashing sized from min/max) vs the
CPU oracle: the Q15 revenue view (GROUP BY l_suppkey) against the
brute-force loop, and random tables with epsilon, clustered and uniform keys
against the interpreter's Fig 10/11 program (Partition over the key's whole
range -> Scatter -> Fold* -> FoldSelect compaction)."""
import numpy as np
import pytest
import torch

import gen
import oracle
from paper_journals_pvldb_pirkmzm16_b200 import vd

pytestmark = pytest.mark.gpu


def load(cols_np):
    keep, views = [], []
    for a in cols_np:
        d = torch.empty(a.size, dtype=torch.from_numpy(a[:0].copy()).dtype, device="cuda")
        views.append(vd.load_column(a, d, compute_minmax=True))
        keep.append(d)
    torch.cuda.synchronize()
    return keep, views


def run_group(views, n, key_col, aggs, pred_=None, float_aggs=()):
    k = views[key_col]
    D = k.max - k.min + 1
    keys = torch.empty(D, dtype=torch.int64, device="cuda")
    rows = torch.empty(D, dtype=torch.int64, device="cuda")
    slots = torch.empty(max(1, D * len(aggs) * 16), dtype=torch.uint8, device="cuda")
    ng = torch.empty(1, dtype=torch.int64, device="cuda")
    vd.group_fold(views, n, key_col, aggs, pred_, out_keys=keys, out_aggs=slots, out_rows=rows, out_ngroups=ng)
    launches = vd.last_launch_count()
    torch.cuda.synchronize()
    g = int(ng.item())
    vals = vd.decode_group_slots(slots[:g * len(aggs) * 16].cpu().numpy().tobytes(), g, len(aggs), float_aggs)
    return keys[:g].cpu().numpy(), vals, rows[:g].cpu().numpy(), launches


Q15_D0, Q15_D1 = 9496, 9587  # [1996-01-01, 1996-04-01) [ext: TPC-H Q15 default DATE]


@pytest.mark.parametrize("n", [1, 1000, 300007])
def test_q15_revenue_view_vs_oracle(n):
    sf = 0.05
    li = {k: gen.host(c, n, sf=sf) for k, c in gen.LINEITEM_COLS.items()}
    exp = oracle.q15(li, Q15_D0, Q15_D1)
    cols = ["l_shipdate", "l_suppkey", "l_extendedprice", "l_discount"]
    keep, views = load([li[c] for c in cols])
    p = vd.pred([[(0, ">=", Q15_D0), (0, "<", Q15_D1)]])
    keys, vals, rows, nl = run_group(views, n, 1, [("sum", [2, (3, 100, -1)]), ("count",)], p)
    got = {int(k): (v[0], v[1]) for k, v in zip(keys, vals)}
    assert got == exp
    assert all(int(r) == v[1] for r, v in zip(rows, vals))  # row count == COUNT(*)
    assert list(keys) == sorted(keys)                       # ascending key order (A16)


@pytest.mark.parametrize("clustered", [False, True])
@pytest.mark.parametrize("D", [1, 4095, 20011])
def test_group_fold_vs_interpreter(clustered, D):
    """Epsilon in the key, the values and the predicate column; integer SUM of
    a column and of a product, MIN, MAX, COUNT, a float SUM (1e-9 relative);
    keys uniform over [kmin, kmin + D) or in runs of equal adjacent keys
    (the warp-combined path)."""
    n = 120013
    rng = np.random.default_rng(D + clustered)
    kmin = -5000
    if clustered:
        k = np.sort(rng.integers(0, D, n)).astype(np.int64) + kmin
    else:
        k = rng.integers(0, D, n).astype(np.int64) + kmin
    k[0], k[-1] = kmin, kmin + D - 1  # metadata spans the whole domain
    v = rng.integers(-10**9, 10**9, n).astype(np.int64)
    w = rng.integers(-100, 100, n).astype(np.int32)
    f = rng.random(n)
    t = rng.integers(0, 100, n).astype(np.int32)
    ek, ev, ew, et = (rng.random(n) < 0.01 for _ in range(4))
    ek[0] = ek[-1] = False
    k[ek], v[ev], w[ew], t[et] = -2**63, -2**63, -2**31, -2**31
    keep, views = load([k, v, w, f, t])
    p = vd.pred([[(4, ">", 9)]])
    aggs = [("sum", [1]), ("sum", [1, 2]), ("min", [1]), ("max", [1]), ("count",), ("sum", [3])]
    keys, vals, rows, nl = run_group(views, n, 0, aggs, p, float_aggs=[False] * 5 + [True])
    assert nl == 5  # init, fold, chunk counts, scan, emit
    po = oracle.run("""
        keep := Greater(t.t, 9)
        positions := FoldSelect(keep)
        sel := Gather(t, positions)
        g := Subtract(sel.k, {kmin})
        prod := Multiply(sel.v, sel.w)
        vals := Zip(g, sel.v, prod, sel.f)
        pivot := Range(0, {D}, 1)
        ppos := Partition(g, pivot)
        sc := Scatter(vals, vals, ppos)
        s_v := FoldSum(sc.g, sc.v)
        s_p := FoldSum(sc.g, sc.prod)
        mn := FoldMin(sc.g, sc.v)
        mx := FoldMax(sc.g, sc.v)
        cnt := FoldCount(sc.g, sc.g)
        s_f := FoldSum(sc.g, sc.f)
        gkey := FoldMax(sc.g, sc.g)
        gpos := FoldSelect(cnt)
        o_key := Gather(gkey, gpos)
        o_sv := Gather(s_v, gpos)
        o_sp := Gather(s_p, gpos)
        o_mn := Gather(mn, gpos)
        o_mx := Gather(mx, gpos)
        o_cnt := Gather(cnt, gpos)
        o_sf := Gather(s_f, gpos)
        """.format(kmin=kmin, D=D), t__k=(k, ek), t__v=(v, ev), t__w=(w, ew), t__f=f, t__t=(t, et))
    ok = [x for x in po.get("o_key") if x is not None]
    assert [int(x) - kmin for x in keys] == ok
    exp_cols = [po.get(c)[:len(ok)] for c in ["o_sv", "o_sp", "o_mn", "o_mx", "o_cnt"]]
    sf_ = po.get("o_sf")[:len(ok)]
    for j in range(len(ok)):
        sv, sp, mn, mx, cnt = (e[j] for e in exp_cols)
        got = vals[j]
        assert got[0] == (sv or 0) and got[1] == (sp or 0)
        assert got[2] == (mn if mn is not None else -2**63)  # all-epsilon group: epsilon (A5)
        assert got[3] == (mx if mx is not None else -2**63)
        assert got[4] == cnt == int(rows[j])
        assert abs(got[5] - sf_[j]) <= 1e-9 * abs(sf_[j]) + 1e-300


def test_group_fold_overflow_and_domain_errors():
    """Without metadata the domain cannot be sized (VD_E_DOMAIN); an integer
    SUM whose exactness the metadata cannot prove is refused (VD_E_OVERFLOW)."""
    k = np.arange(1000, dtype=np.int64)
    v = np.full(1000, 2**62, dtype=np.int64)
    keep, views = load([k, v])
    with pytest.raises(vd.VdError) as e:
        run_group(views, 1000, 0, [("sum", [1])])
    assert e.value.status == vd.VD_E_OVERFLOW
    views[0].has_minmax = 0
    with pytest.raises(vd.VdError) as e:
        run_group(views, 1000, 0, [("count",)])
    assert e.value.status == vd.VD_E_DOMAIN
