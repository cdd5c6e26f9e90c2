"""GPU parity of vd_hash_group_fold (grouped fold over
SPARSE keys -- open-addressing tables sized from a distinct-key bound,
shared-memory tables spilling to a global one) and vd_merge_groups (the
cross-GPU merge of compacted groups) against the oracle.

The sparse keys are an injective remapping of l_suppkey onto 64-bit values
(multiplication by an odd constant mod 2^64: a bijection), so the expected
groups are the oracle's Q15 program / brute-force loop on the dense
l_suppkey, re-keyed -- the grouping result is invariant under a renaming of
the keys.  Hash tables have no key order, so groups are compared as a
mapping and checked to occur exactly once."""
import numpy as np
import pytest
import torch

import gen
import oracle
from oracle import programs
from paper_journals_pvldb_pirkmzm16_b200 import vd

pytestmark = pytest.mark.gpu

Q15_D0, Q15_D1 = 9496, 9587
MULT = 0x9E3779B97F4A7C15  # odd: k -> k * MULT mod 2^64 is injective


def sparse(keys32):
    k = (keys32.astype(np.uint64) * np.uint64(MULT)).view(np.int64)
    assert (k != np.int64(-2**63)).all()  # never the epsilon sentinel
    return k


def rekey(k):
    return int(sparse(np.array([k], dtype=np.int64))[0])


def run_hash(views, n, key_col, aggs, pred_, max_groups, float_aggs=()):
    cap = max_groups
    keys = torch.empty(cap, dtype=torch.int64, device="cuda")
    rows = torch.empty(cap, dtype=torch.int64, device="cuda")
    slots = torch.empty(max(1, cap * len(aggs) * 16), dtype=torch.uint8, device="cuda")
    ng = torch.empty(1, dtype=torch.int64, device="cuda")
    vd.hash_group_fold(views, n, key_col, aggs, pred_, max_groups=max_groups, out_keys=keys, out_aggs=slots,
                       out_rows=rows, out_ngroups=ng)
    torch.cuda.synchronize()
    g = int(ng.item())
    assert g >= 0, "table full"
    vals = vd.decode_group_slots(slots[:g * len(aggs) * 16].cpu().numpy().tobytes(), g, len(aggs), float_aggs)
    return keys[:g], slots[:g * len(aggs) * 16], rows[:g], g, keys[:g].cpu().numpy(), vals, rows[:g].cpu().numpy()


def q15_li(n, sf=0.05):
    li = {k: gen.host(c, n, sf=sf) for k, c in gen.LINEITEM_COLS.items()}
    li["l_skey"] = sparse(li["l_suppkey"])
    return li


@pytest.mark.parametrize("n", [1, 5000, 300007])
def test_hash_q15_sparse_keys_vs_bruteforce(n):
    li = q15_li(n)
    exp = {rekey(k): v for k, v in oracle.q15(li, Q15_D0, Q15_D1).items()}
    cols = ["l_shipdate", "l_skey", "l_extendedprice", "l_discount"]
    keep = [torch.from_numpy(li[c]).cuda() for c in cols]
    views = [vd.describe(t) for t in keep]
    p = vd.pred([[(0, ">=", Q15_D0), (0, "<", Q15_D1)]])
    *_, keys, vals, rows = run_hash(views, n, 1, [("sum", [2, (3, 100, -1)]), ("count",)], p, max_groups=20000)
    got = {int(k): (v[0], v[1]) for k, v in zip(keys, vals)}
    assert len(got) == len(keys)  # every group exactly once
    assert got == exp
    assert all(int(r) == v[1] for r, v in zip(rows, vals))


def test_hash_q15_vs_interpreter_program_with_remapped_keys():
    """The interpreter's Q15 program (Fig 10/11 chain: Partition over the
    dense key range -> Scatter -> FoldSum/FoldCount -> FoldSelect) on the
    dense keys, re-keyed, equals the hash fold on the sparse keys."""
    n = 60001
    li = q15_li(n, sf=0.02)
    kmin = int(li["l_suppkey"].min())
    D = int(li["l_suppkey"].max()) - kmin + 1
    p = oracle.Program()
    for c in ("l_shipdate", "l_suppkey", "l_extendedprice", "l_discount"):
        p.set("lineitem." + c, li[c])
    p.run(programs.Q15.format(d0m1=Q15_D0 - 1, d1=Q15_D1, kmin=kmin, D=D))
    exp = {rekey(k + kmin): (r, c) for k, r, c in zip(p.get("o_key"), p.get("o_rev"), p.get("o_cnt"))
           if k is not None}
    cols = ["l_shipdate", "l_skey", "l_extendedprice", "l_discount"]
    keep = [torch.from_numpy(li[c]).cuda() for c in cols]
    views = [vd.describe(t) for t in keep]
    pr = vd.pred([[(0, ">=", Q15_D0), (0, "<", Q15_D1)]])
    *_, keys, vals, rows = run_hash(views, n, 1, [("sum", [2, (3, 100, -1)]), ("count",)], pr, max_groups=4096)
    assert {int(k): (v[0], v[1]) for k, v in zip(keys, vals)} == exp


@pytest.mark.parametrize("nkeys", [3, 900, 200000])
def test_hash_epsilon_min_max_and_spill(nkeys):
    """Few keys (all in the shared tables), ~1 shared table's worth, and far
    more than a shared table holds (spill to the global table); epsilon
    keys / values; MIN, MAX, integer SUM of a product, f64 SUM, COUNT --
    against a pandas group-by over the non-epsilon rows."""
    import pandas as pd
    n = 250007
    rng = np.random.default_rng(nkeys)
    kd = rng.integers(0, nkeys, n)
    k = sparse(kd)
    k[rng.random(n) < 0.01] = -2**63  # epsilon key: no group
    v = rng.integers(-10**6, 10**6, n).astype(np.int64)
    ev = rng.random(n) < 0.02
    v[ev] = -2**63
    f = rng.random(n)
    dk, dv, df = (torch.from_numpy(a).cuda() for a in (k, v, f))
    views = [vd.column(dk), vd.column(dv, minmax=(-10**6, 10**6)), vd.column(df)]
    aggs = [("sum", [1, (1, 0, 1)]), ("min", [1]), ("max", [1]), ("sum", [2]), ("count",)]
    *_, keys, vals, rows = run_hash(views, n, 0, aggs, None, max_groups=max(nkeys, 1) + 10,
                                    float_aggs=[False, False, False, True])
    df_ = pd.DataFrame({"k": k, "v": v, "ev": ev, "f": f})
    df_ = df_[df_.k != -2**63]
    vv = df_[~df_.ev]
    exp_sum = vv.groupby("k")["v"].apply(lambda s: int(sum(int(x) * int(x) for x in s)))
    exp_min, exp_max = vv.groupby("k")["v"].min(), vv.groupby("k")["v"].max()
    exp_f, exp_cnt = df_.groupby("k")["f"].sum(), df_.groupby("k").size()
    assert len(keys) == len(exp_cnt) == len(set(keys.tolist()))
    for kk, vals_, r in zip(keys.tolist(), vals, rows.tolist()):
        assert vals_[0] == exp_sum.get(kk, 0)
        assert vals_[1] == (int(exp_min[kk]) if kk in exp_min.index else -2**63)
        assert vals_[2] == (int(exp_max[kk]) if kk in exp_max.index else -2**63)
        assert abs(vals_[3] - exp_f[kk]) <= 1e-9 * max(1.0, abs(exp_f[kk]))
        assert vals_[4] == r == int(exp_cnt[kk])


def test_hash_table_full_reports_minus_one():
    n = 100000
    k = sparse(np.arange(n, dtype=np.int64))
    dk = torch.from_numpy(k).cuda()
    keys = torch.empty(1, dtype=torch.int64, device="cuda")
    ng = torch.empty(1, dtype=torch.int64, device="cuda")
    big = torch.empty(n, dtype=torch.int64, device="cuda")
    vd.hash_group_fold([vd.column(dk)], n, 0, [("count",)], None, max_groups=100, out_keys=big,
                       out_aggs=torch.empty(n * 16, dtype=torch.uint8, device="cuda"), out_rows=big.clone(),
                       out_ngroups=ng)
    torch.cuda.synchronize()
    assert int(ng.item()) == -1


@pytest.mark.parametrize("G", [2, 3, 8])
def test_merge_groups_of_shards_equals_whole(G):
    """The cross-GPU merge of compacted groups (vd_merge_groups): each
    'rank' hash-folds its row range, the G outputs are concatenated (as an
    all-gather leaves them) and merged; the result equals the whole-table
    oracle (pin P8: shards merge to the whole) with 128-bit sums."""
    n = 300007
    li = q15_li(n)
    exp = {rekey(k): v for k, v in oracle.q15(li, Q15_D0, Q15_D1).items()}
    cols = ["l_shipdate", "l_skey", "l_extendedprice", "l_discount"]
    keep = [torch.from_numpy(li[c]).cuda() for c in cols]
    views = [vd.describe(t) for t in keep]
    p = vd.pred([[(0, ">=", Q15_D0), (0, "<", Q15_D1)]])
    aggs = [("sum", [2, (3, 100, -1)]), ("count",)]
    # every "rank" writes into its block of fixed stride (an all-gather of
    # fixed-size buffers leaves them so), its group count into counts[r]
    stride = 20000
    allk = torch.zeros(G * stride, dtype=torch.int64, device="cuda")
    allr = torch.zeros(G * stride, dtype=torch.int64, device="cuda")
    alls = torch.zeros(G * stride * 2 * 16, dtype=torch.uint8, device="cuda")
    counts = torch.zeros(G, dtype=torch.int64, device="cuda")
    for r in range(G):
        a, b = r * n // G, (r + 1) * n // G
        sv = [vd.column(t[a:b], minmax=(v.min, v.max), noeps=bool(v.flags & vd.VD_COL_NOEPS))
              for t, v in zip(keep, views)]
        vd.hash_group_fold(sv, b - a, 1, aggs, p, max_groups=stride, out_keys=allk[r * stride:(r + 1) * stride],
                           out_aggs=alls[r * stride * 32:(r + 1) * stride * 32],
                           out_rows=allr[r * stride:(r + 1) * stride], out_ngroups=counts[r:r + 1])
    ok = torch.empty(stride, dtype=torch.int64, device="cuda")
    orows = torch.empty(stride, dtype=torch.int64, device="cuda")
    oslots = torch.empty(stride * 2 * 16, dtype=torch.uint8, device="cuda")
    ong = torch.empty(1, dtype=torch.int64, device="cuda")
    vd.merge_groups(allk, alls, allr, counts, G, stride, [vd.VD_AGG_SUM, vd.VD_AGG_COUNT], [False, False],
                    max_groups=stride, out_keys=ok, out_aggs=oslots, out_rows=orows, out_ngroups=ong)
    torch.cuda.synchronize()
    g = int(ong.item())
    vals = vd.decode_group_slots(oslots[:g * 32].cpu().numpy().tobytes(), g, 2)
    got = {int(k): (v[0], v[1]) for k, v in zip(ok[:g].cpu().tolist(), vals)}
    assert got == exp
    assert orows[:g].cpu().tolist() == [v[1] for v in vals]
