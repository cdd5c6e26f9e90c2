"""GPU parity of the fused pipelines (vd_run_pipeline) vs the CPU oracle.

Each plan runs through its specialised fragment and through the generic
fragment (force_generic), in branching and predicated mode, on generated
TPC-H-shaped tables that span many tiles with a ragged tail; integer /
decimal aggregates bit-exact, the f64 selective sum within 1e-9 relative.
"""
import contextlib
import os

import numpy as np
import pytest
import torch

import gen
import oracle
from paper_journals_pvldb_pirkmzm16_b200 import plans, vd

pytestmark = pytest.mark.gpu


def load(cols_np):
    """a1: vd_load_column for each host column (min/max metadata computed)."""
    keep, views = [], []
    for a in cols_np:
        d = torch.empty(a.size, dtype=torch.from_numpy(a[:0].copy()).dtype, device="cuda")
        views.append(vd.load_column(a, d, compute_minmax=True))
        keep.append(d)
    torch.cuda.synchronize()
    return keep, views


def run(plan, views, n, dims=(), want=None):
    out = torch.empty(vd.partials_bytes(plan), dtype=torch.uint8, device="cuda")
    vd.run_pipeline(plan, views, n, dims, out=out)
    launches = vd.last_launch_count()
    frag = vd.last_fragment()
    torch.cuda.synchronize()
    if want is not None:
        assert frag in want, (frag, want)
    return out.cpu().numpy().tobytes(), launches


@contextlib.contextmanager
def env(**kv):
    """Set dispatch environment variables for the duration of a block."""
    old = {k: os.environ.get(k) for k in kv}
    os.environ.update(kv)
    try:
        yield
    finally:
        for k, v in old.items():
            if v is None:
                os.environ.pop(k, None)
            else:
                os.environ[k] = v


def lineitem(sf, n=None, seed=gen.DEFAULT_SEED):
    n = gen.lineitem_rows(sf) if n is None else n
    return {k: gen.host(c, n, sf=sf, seed=seed, threads=8) for k, c in gen.LINEITEM_COLS.items()}


@pytest.mark.parametrize("sel_mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED])
@pytest.mark.parametrize("generic", [False, True])
@pytest.mark.parametrize("n", [1, 7, 4099, 60001, 600003])
def test_q1_vs_oracle(sel_mode, generic, n):
    li = lineitem(0.1, n)
    exp = oracle.q1(li)
    keep, views = load([li[c] for c in plans.Q1_COLS])
    plan = plans.q1(sel_mode, force_generic=generic)
    buf, nl = run(plan, views, n, want=("generic",) if generic else ("q1_tma",))
    got = vd.decode_partials(buf, plan)
    assert {k: v[:6] for k, v in got.items()} == exp
    for k, v in got.items():
        assert v[6] == v[5]  # row count slot == count(*) aggregate
    assert nl == 1  # one fused kernel per pipeline call


def test_q1_key_domain_proof_and_ship_edge():
    """All rows on the predicate edge (ship == 10471 kept, 10472 dropped)."""
    n = 10000
    li = lineitem(0.01, n)
    li["l_shipdate"][:] = 10471
    li["l_shipdate"][::2] = 10472
    exp = oracle.q1(li)
    keep, views = load([li[c] for c in plans.Q1_COLS])
    for generic in [False, True]:
        plan = plans.q1(force_generic=generic)
        got = vd.decode_partials(run(plan, views, n)[0], plan)
        assert {k: v[:6] for k, v in got.items()} == exp


def test_q1_unaligned_columns_fall_back_exactly():
    """Column views at odd offsets cannot use 16-byte loads: the planner falls
    back and the result is unchanged."""
    n = 50001
    li = lineitem(0.1, n + 1)
    exp = oracle.q1({k: v[1:] for k, v in li.items()})
    keep, views = load([li[c] for c in plans.Q1_COLS])
    shifted = []
    for v, c in zip(views, plans.Q1_COLS):
        w = vd.vd_column.from_buffer_copy(v)
        w.data = v.data + li[c].itemsize
        w.len = n
        shifted.append(w)
    plan = plans.q1()
    buf, nl = run(plan, shifted, n)
    got = vd.decode_partials(buf, plan)
    assert {k: v[:6] for k, v in got.items()} == exp


@pytest.mark.parametrize("sel_mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED])
@pytest.mark.parametrize("generic", [False, True])
@pytest.mark.parametrize("n", [3, 4096, 600007])
def test_q6_vs_oracle(sel_mode, generic, n):
    li = lineitem(0.1, n)
    rev, cnt = oracle.q6(li)
    keep, views = load([li[c] for c in plans.Q6_COLS])
    plan = plans.q6(sel_mode, force_generic=generic)
    buf, nl = run(plan, views, n, want=("generic",) if generic else ("scalar_tma",))
    got = vd.decode_partials(buf, plan)
    if cnt == 0:
        assert got == {}
    else:
        assert got == {0: [rev, cnt, cnt]}
    assert nl == 1
    if sel_mode == vd.VD_SEL_BRANCH and not generic:
        with env(VD_LATE="force"):  # late loads: l_shipdate leads, the rest per qualifying row
            assert vd.decode_partials(run(plan, views, n, want=("late",))[0], plan) == got


@pytest.mark.parametrize("sel_mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED])
@pytest.mark.parametrize("generic", [False, True])
@pytest.mark.parametrize("n", [5, (1 << 20) + 3])
def test_selective_sum_f32_vs_oracle(sel_mode, generic, n):
    """C1 shape: select v < 0.5, FoldSum of the selected f32 values in f64."""
    v = gen.host(gen.F32_UNIFORM, n, seed=21)
    t = float(np.float32(0.5))
    _, c, (sh, sl) = oracle.select_f32(v, t, "lt", want_positions=False)
    keep, views = load([v])
    plan = plans.selsum(t, sel_mode, force_generic=generic)
    buf, nl = run(plan, views, n, want=("generic",) if generic else ("selsum_tma",))
    got = vd.decode_partials(buf, plan, float_aggs=[True, False])
    assert got[0][1] == c
    ref = sh + sl
    assert abs(got[0][0] - ref) <= 1e-9 * abs(ref)


def _dims(sf):
    part = {k: gen.host(c, gen.part_rows(sf), sf=sf) for k, c in gen.PART_COLS.items()}
    supp = {k: gen.host(c, gen.supplier_rows(sf), sf=sf) for k, c in gen.SUPPLIER_COLS.items()}
    return part, supp


def codes():
    return {"brand": {s: i for i, s in enumerate(gen.BRAND)},
            "container": {s: i for i, s in enumerate(gen.CONTAINER)},
            "shipmode": {s: i for i, s in enumerate(gen.SHIPMODE)},
            "shipinstruct": {s: i for i, s in enumerate(gen.SHIPINSTRUCT)}}


@pytest.mark.parametrize("sel_mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED])
@pytest.mark.parametrize("generic", [False, True])
@pytest.mark.parametrize("n", [None, 100003])
def test_fkj_q19_vs_oracle(sel_mode, generic, n):
    sf = 0.05
    li = lineitem(sf, n)
    part, supp = _dims(sf)
    exp = oracle.fkj(0, li, part, supp)
    keep, views = load([li[c] for c in plans.Q19_COLS])
    dkeep, dviews = load([part[c] for c in plans.Q19_DIMS])
    plan = plans.q19(codes(), sel_mode, force_generic=generic)
    frag = ("generic",) if generic else (("late",) if sel_mode == vd.VD_SEL_BRANCH else ("star_join",))
    got = vd.decode_partials(run(plan, views, len(li["l_partkey"]), dviews, want=frag)[0], plan)
    assert {k: tuple(v[:2]) for k, v in got.items()} == exp
    if sel_mode == vd.VD_SEL_BRANCH and not generic:
        with env(VD_LATE_FAST="0"):  # the late fragment without its fast first round
            got = vd.decode_partials(run(plan, views, len(li["l_partkey"]), dviews, want=("late",))[0], plan)
        assert {k: tuple(v[:2]) for k, v in got.items()} == exp
        with env(VD_LATE="off"):  # the dense star-join fragment on the same plan
            got = vd.decode_partials(run(plan, views, len(li["l_partkey"]), dviews, want=("star_join",))[0], plan)
        assert {k: tuple(v[:2]) for k, v in got.items()} == exp


def test_fkj_q19_gather_fold_fragment():
    """The Q19 plan through the general gather-fold fragment (star-join off)."""
    import os
    sf = 0.05
    li = lineitem(sf, 300007)
    part, supp = _dims(sf)
    exp = oracle.fkj(0, li, part, supp)
    keep, views = load([li[c] for c in plans.Q19_COLS])
    dkeep, dviews = load([part[c] for c in plans.Q19_DIMS])
    with env(VD_STAR_VARIANT="off", VD_LATE="off"):
        got = vd.decode_partials(run(plans.q19(codes()), views, len(li["l_partkey"]), dviews,
                                     want=("gather_fold",))[0], plans.q19(codes()))
    assert {k: tuple(v[:2]) for k, v in got.items()} == exp


def _term_expr(name, col, cmp, c, out):
    """A predicate term as the oracle's Greater/Equals/LogicalOr (reading A8)."""
    if cmp == ">":
        out.append(f"{name} := Greater({col}, {c})")
    elif cmp == "<":
        out.append(f"{name} := Greater({c}, {col})")
    elif cmp == "==":
        out.append(f"{name} := Equals({col}, {c})")
    elif cmp == ">=":
        out.append(f"{name} := Greater({col}, {c - 1})")
    elif cmp == "<=":
        out.append(f"{name} := Greater({c + 1}, {col})")
    elif cmp == "!=":
        out += [f"{name}_a := Greater({col}, {c})", f"{name}_b := Greater({c}, {col})",
                f"{name} := LogicalOr({name}_a, {name}_b)"]
    else:  # in: c is a list of codes
        codes = c or [1000]  # the empty set: never equal
        out.append(f"{name} := Equals({col}, {codes[0]})")
        for k, v in enumerate(codes[1:]):
            out += [f"{name}_{k} := Equals({col}, {v})", f"{name} := LogicalOr({name}, {name}_{k})"]


@pytest.mark.parametrize("seed", range(12))
def test_star_join_random_predicates_vs_oracle(seed):
    """Star-join fragment on random disjunctive predicates over its slot
    columns (every comparison kind, dictionary codes >= 64, epsilon in every
    column, FKs outside the dimension, conjunctions without dimension terms)
    against the oracle: each conjunction's FoldSelect positions from an oracle
    program (a term over epsilon is false, A9), their union, then the oracle's
    Gather -> Multiply -> FoldSum / FoldCount over it."""
    rng = np.random.default_rng(100 + seed)
    n, m = 70001 + seed * 997, 3001
    fk = rng.integers(-3, m + 5, n).astype(np.int32)
    rq = rng.integers(0, 6000, n).astype(np.int64)
    u1 = rng.integers(0, 90, n).astype(np.uint8)
    u2 = rng.integers(0, 8, n).astype(np.uint8)
    x = rng.integers(0, 10**7, n).astype(np.int64)
    y = rng.integers(0, 11, n).astype(np.int64)
    d1 = rng.integers(0, 80, m).astype(np.uint8)
    d2 = rng.integers(0, 40, m).astype(np.uint8)
    dr = rng.integers(1, 51, m).astype(np.int32)
    eps = {}
    for nm, arr, e in [("fk", fk, -2**31), ("rq", rq, -2**63), ("u1", u1, 255), ("u2", u2, 255), ("x", x, -2**63),
                       ("y", y, -2**63), ("d1", d1, 255), ("d2", d2, 255), ("dr", dr, -2**31)]:
        msk = rng.random(arr.size) < 0.01
        arr[msk] = e
        eps[nm] = msk
    base = {"fk": fk, "rq": rq, "x": x, "y": y, "u1": u1, "u2": u2}  # plan column order
    cols = list(base)
    slot_ref = {"rq": 1, "u1": 4, "u2": 5, "d1": 6, "d2": 7, "dr": 8}

    def rand_term(colname):
        if colname in ("u1", "u2", "d1", "d2"):
            cmp = str(rng.choice([">", "<", "==", ">=", "<=", "!=", "in"], p=[.17, .17, .04, .17, .17, .14, .14]))
            if cmp == "in":
                return cmp, sorted(set(int(v) for v in rng.integers(0, 64, rng.integers(0, 60))))
            return cmp, int(rng.integers(0, 90))
        hi = 6000 if colname == "rq" else 50
        return str(rng.choice([">", "<", "==", ">=", "<="], p=[.3, .3, .05, .175, .175])), int(rng.integers(0, hi))

    nconj = int(rng.integers(1, 5))
    conjs = []
    for c in range(nconj):
        names = [k for k in slot_ref if rng.random() < 0.4] or ["u2"]
        if c == 0:
            names = sorted(set(names) | {"u1", "rq", "d1", "dr"})
        conjs.append([(k, *rand_term(k)) for k in names for _ in range(1 + int(rng.random() < 0.2))][:8])
    # the oracle: one program per conjunction, union of the selected positions
    sel = np.zeros(n, dtype=bool)
    inputs = {f"fact__{k}": (v, eps[k]) for k, v in base.items()}
    inputs.update({f"dim__{k}": (v, eps[k]) for k, v in (("d1", d1), ("d2", d2), ("dr", dr))})
    for c, terms in enumerate(conjs):
        lines = ["p := Subtract(fact.fk, 1)", "gd1 := Gather(dim.d1, p)", "gd2 := Gather(dim.d2, p)",
                 "gdr := Gather(dim.dr, p)"]
        ref = {"rq": "fact.rq", "u1": "fact.u1", "u2": "fact.u2", "d1": "gd1", "d2": "gd2", "dr": "gdr"}
        names = []
        for k, (colname, cmp, val) in enumerate(terms):
            _term_expr(f"t{k}", ref[colname], cmp, val, lines)
            names.append(f"t{k}")
        lines.append(f"a := LogicalAnd({names[0]}, {names[0]})")
        for nm in names[1:]:
            lines.append(f"a := LogicalAnd(a, {nm})")
        lines.append("pos := FoldSelect(a)")
        pos, pe = oracle.run("\n".join(lines), **inputs).get_arrays("pos")
        sel[pos[~pe]] = True
    upos = np.nonzero(sel)[0].astype(np.int64)
    agg = oracle.run("""
    gx := Gather(fact.x, pos)
    gy := Gather(fact.y, pos)
    f := Multiply(gy, -1)
    t := Add(f, 100)
    pr := Multiply(gx, t)
    s := FoldSum(pr)
    c := FoldCount(pos)
    """, fact__x=(x, eps["x"]), fact__y=(y, eps["y"]), pos=upos)
    exp_s, exp_c = (agg.get("s")[0], agg.get("c")[0]) if upos.size else (0, 0)
    # the GPU plan
    vconj = []
    for terms in conjs:
        ts = []
        for colname, cmp, val in terms:
            if cmp == "in":
                ts.append((slot_ref[colname], "in", val))
            else:
                ts.append((slot_ref[colname], str(cmp), val))
        vconj.append(ts)
    keep, views = load([base[k] for k in cols])
    dkeep, dviews = load([d1, d2, dr])
    plan = vd.pipeline(pred_=vd.pred(vconj), gathers=[(0, 0, 1), (0, 1, 1), (0, 2, 1)],
                       aggs=[("sum", [2, (3, 100, -1)]), ("count",)])
    with env(VD_LATE="off"):
        got = vd.decode_partials(run(plan, views, n, dviews, want=("star_join",))[0], plan)
    if exp_c == 0:
        assert got == {}
    else:
        assert got == {0: [int(exp_s), int(exp_c), int(exp_c)]}
    # default dispatch (the late-materialisation fragment when the conjunctions
    # share interval terms on u8 / i32 columns) and the general gather-fold one
    assert vd.decode_partials(run(plan, views, n, dviews, want=("star_join", "late"))[0], plan) == got
    with env(VD_LATE="off", VD_STAR_VARIANT="off"):
        assert vd.decode_partials(run(plan, views, n, dviews, want=("gather_fold",))[0], plan) == got
    gen_plan = vd.pipeline(pred_=vd.pred(vconj), gathers=[(0, 0, 1), (0, 1, 1), (0, 2, 1)],
                           aggs=[("sum", [2, (3, 100, -1)]), ("count",)], force_generic=True)
    assert vd.decode_partials(run(gen_plan, views, n, dviews, want=("generic",))[0], gen_plan) == got


@pytest.mark.parametrize("sel_mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED])
@pytest.mark.parametrize("generic", [False, True])
@pytest.mark.parametrize("n", [None, 100003])
def test_fkj_q9_vs_oracle(sel_mode, generic, n):
    sf = 0.05
    li = lineitem(sf, n)
    part, supp = _dims(sf)
    exp = oracle.fkj(1, li, part, supp)
    keep, views = load([li[c] for c in plans.Q9_COLS])
    dkeep, dviews = load([supp[c] for c in plans.Q9_DIMS])
    plan = plans.q9(sel_mode, force_generic=generic)
    got = vd.decode_partials(run(plan, views, len(li["l_suppkey"]), dviews,
                                 want=("generic",) if generic else ("fk_group",))[0], plan)
    assert {k: tuple(v[:2]) for k, v in got.items()} == exp


@pytest.mark.parametrize("variant", ["fk_group_priv", "fk_group_priv_checked", "fk_group"])
@pytest.mark.parametrize("n", [1023, 1024, 70001])
def test_fkj_q9_fk_group_variants(variant, n):
    """The Q9 FK grouped fold through each of its kernels: private slots with
    the checks proven away (metadata with VD_COL_NOEPS), private slots with
    per-row checks (no epsilon metadata), shared-memory atomics."""
    import os
    sf = 0.05
    li = lineitem(sf, n)
    part, supp = _dims(sf)
    exp = oracle.fkj(1, li, part, supp)
    keep, views = load([li[c] for c in plans.Q9_COLS])
    dkeep, dviews = load([supp[c] for c in plans.Q9_DIMS])
    if variant != "fk_group_priv":
        for v in views + dviews:
            v.flags = 0
    plan = plans.q9()
    if variant != "fk_group":
        os.environ["VD_FKG_VARIANT"] = "priv"
    try:
        got = vd.decode_partials(run(plan, views, n, dviews, want=(variant,))[0], plan)
    finally:
        os.environ.pop("VD_FKG_VARIANT", None)
    assert {k: tuple(v[:2]) for k, v in got.items()} == exp


@pytest.mark.parametrize("variant", ["fk_group_priv_checked", "fk_group", "generic"])
def test_fkj_q9_epsilon_vs_interpreter(variant):
    """Q9 with epsilon everywhere, against the oracle's Voodoo program (Fig
    10/11 shape): an epsilon or out-of-range l_suppkey gathers epsilon
    (A11), an epsilon nation or ship date makes the key epsilon -- the row
    has no group (A9, Partition drops it) -- and an epsilon l_extendedprice
    or l_discount makes the row's revenue epsilon: skipped by the SUM (A5)
    but the row still counts (COUNT(*) = FoldCount over the key)."""
    import datetime
    import os
    sf = 0.05
    n = 100003
    li = lineitem(sf, n)
    part, supp = _dims(sf)
    rng = np.random.default_rng(11)
    eps = {c: rng.random(n) < 0.01 for c in plans.Q9_COLS}
    for c, e in eps.items():
        li[c] = li[c].copy()
        li[c][e] = {"i": -2**31 if li[c].dtype == np.int32 else -2**63}[li[c].dtype.kind]
    oob = rng.random(n) < 0.005
    li["l_suppkey"][oob & ~eps["l_suppkey"]] = len(supp["s_nationkey"]) + 5
    nat = supp["s_nationkey"].copy()
    enat = rng.random(len(nat)) < 0.02
    nat[enat] = 0xFF
    day0 = 8035
    cal = np.array([(datetime.date(1970, 1, 1) + datetime.timedelta(days=day0 + i)).year for i in range(3000)])
    p = oracle.Program()
    for c in plans.Q9_COLS:
        p.set("lineitem." + c, li[c], eps[c])
    p.set("supplier.s_nationkey", nat, enat)
    p.set("calendar.year", cal)
    p.run(__import__("oracle.programs", fromlist=["x"]).FKJ_Q9.format(day0=day0)
          + "rows := FoldCount(sc.g, sc.g)\no_rows := Gather(rows, gpos)\n")
    keys = p.get("o_key")
    exp = {k: (p.get("o_rev")[j] or 0, p.get("o_rows")[j]) for j, k in enumerate(keys) if k is not None}
    keep, views = load([li[c] for c in plans.Q9_COLS])
    dkeep, dviews = load([nat])
    plan = plans.q9(force_generic=(variant == "generic"))
    if variant == "fk_group_priv_checked":
        os.environ["VD_FKG_VARIANT"] = "priv"
    try:
        got = vd.decode_partials(run(plan, views, n, dviews, want=(variant,))[0], plan)
    finally:
        os.environ.pop("VD_FKG_VARIANT", None)
    assert {k: tuple(v[:2]) for k, v in got.items()} == exp


def test_generic_min_max_and_float_products():
    """Generic fragment: MIN/MAX and float aggregates, grouped, with epsilon;
    against the interpreter's Fig 10/11 program (FoldSelect -> Gather ->
    Partition -> Scatter -> FoldMin / FoldMax / FoldSum / FoldCount)."""
    n = 200003
    rng = np.random.default_rng(1)
    k = rng.integers(0, 5, n).astype(np.int32)
    x = rng.integers(-10**9, 10**9, n).astype(np.int64)
    f = rng.random(n)
    x[::97] = -2**63  # epsilon
    keep, views = load([k, x, f])
    plan = vd.pipeline(pred_=vd.pred([[(1, ">", -5 * 10**8)]]), key=[(0, 0, 0, 1)], ngroups=5,
                       aggs=[("min", [1]), ("max", [1]), ("sum", [2, (1, 0, 1)]), ("sum", [(2, 1, 2)]), ("count",)])
    got = vd.decode_partials(run(plan, views, n)[0], plan, float_aggs=[False, False, True, True, False])
    ex = x == -2**63
    p = oracle.Program()
    p.set("t.k", k)
    p.set("t.x", np.where(ex, 0, x), ex)
    p.set("t.f", f)
    p.run("""
keep := Greater(t.x, -500000000)
positions := FoldSelect(keep)
sel := Gather(t, positions)
fx := Multiply(sel.f, sel.x)
f2 := Multiply(sel.f, 2)
g2 := Add(f2, 1)
vals := Zip(sel.k, sel.x, fx, g2)
pivot := Range(0, 5, 1)
ppos := Partition(sel.k, pivot)
sc := Scatter(vals, vals, ppos)
mn := FoldMin(sc.k, sc.x)
mx := FoldMax(sc.k, sc.x)
s1 := FoldSum(sc.k, sc.fx)
s2 := FoldSum(sc.k, sc.g2)
cnt := FoldCount(sc.k, sc.k)
gk := FoldMax(sc.k, sc.k)
gpos := FoldSelect(cnt)
o_k := Gather(gk, gpos)
o_mn := Gather(mn, gpos)
o_mx := Gather(mx, gpos)
o_s1 := Gather(s1, gpos)
o_s2 := Gather(s2, gpos)
o_c := Gather(cnt, gpos)
""")
    keys = p.get("o_k")
    outs = {o: p.get(o) for o in ("o_mn", "o_mx", "o_s1", "o_s2", "o_c")}
    exp = {kk: [outs[o][j] for o in ("o_mn", "o_mx", "o_s1", "o_s2", "o_c")] for j, kk in enumerate(keys)
           if kk is not None}
    assert set(got) == set(exp)
    for g, e in exp.items():
        assert got[g][0] == e[0] and got[g][1] == e[1]
        assert abs(got[g][2] - e[2]) <= 1e-9 * abs(e[2])
        assert abs(got[g][3] - e[3]) <= 1e-9 * abs(e[3])
        assert got[g][4] == e[4] == got[g][5]


def test_virtual_shards_merge_equals_whole_q1():
    """Pin P8 on the GPU: G row-range shards (the ctrl floor(i*G/n) one level
    above CTAs) run separately and merged by vd_merge_partials equal the
    single-shard result and the oracle."""
    n = 600011
    li = lineitem(0.1, n)
    exp = oracle.q1(li)
    keep, views = load([li[c] for c in plans.Q1_COLS])
    plan = plans.q1()
    for G in [2, 3, 8]:
        parts = []
        for r in range(G):
            a, b = r * n // G, (r + 1) * n // G
            sv = []
            for v, c in zip(views, plans.Q1_COLS):
                w = vd.vd_column.from_buffer_copy(v)
                w.data = v.data + a * li[c].itemsize
                w.len = b - a
                sv.append(w)
            parts.append(run(plan, sv, b - a)[0])
        got = vd.merge_partials(plan, views, [], parts)  # rank-order merge + Fig 11 compaction
        assert {k: v[:6] for k, v in got.items()} == exp


@pytest.mark.parametrize("op", [">", ">=", "<", "<=", "=="])
@pytest.mark.parametrize("c", [0.1, float(np.float32(0.5)), 0.75000000000000011])
def test_selective_sum_f32_interval_edges(op, c):
    """The f32 interval form of a single comparison against a double constant
    (x > c <=> x >= succ(floor32(c)), ...) agrees with exact comparisons of
    the f32 values promoted to double (numpy), including the f32 neighbours
    of the constant, epsilon (NaN) and infinities."""
    base = np.float32(c)
    near = [np.nextafter(base, np.float32(-np.inf)), base, np.nextafter(base, np.float32(np.inf))]
    v = np.concatenate([np.array(near * 5000, dtype=np.float32), gen.host(gen.F32_UNIFORM, 100003, seed=5),
                        np.array([np.inf, -np.inf, np.nan, 0.0], dtype=np.float32)])
    keep, views = load([v])
    plan = vd.pipeline(pred_=vd.pred([[(0, op, float(c))]]), aggs=[("sum", [0]), ("count",)])
    buf, _ = run(plan, views, len(v), want=("selsum_tma",))
    got = vd.decode_partials(buf, plan, float_aggs=[True, False])
    x = v.astype(np.float64)
    m = {">": x > c, ">=": x >= c, "<": x < c, "<=": x <= c, "==": x == c}[op] & ~np.isnan(x)
    if m.sum() == 0:
        assert got == {}
        return
    assert got[0][1] == int(m.sum())
    ref = float(np.sum(x[m]))
    assert got[0][0] == ref or abs(got[0][0] - ref) <= 1e-9 * abs(ref)


@pytest.mark.parametrize("variant", ["gather_fold", "generic"])
def test_fkj_q9_gather_fold_fragment(variant):
    """The Q9 plan through the general gather-fold fragment (the FK grouped
    fragment disabled) and through the generic one."""
    import os
    sf = 0.05
    li = lineitem(sf, 200003)
    part, supp = _dims(sf)
    exp = oracle.fkj(1, li, part, supp)
    keep, views = load([li[c] for c in plans.Q9_COLS])
    dkeep, dviews = load([supp[c] for c in plans.Q9_DIMS])
    plan = plans.q9(force_generic=(variant == "generic"))
    os.environ["VD_FKG_VARIANT"] = "off"
    try:
        got = vd.decode_partials(run(plan, views, len(li["l_suppkey"]), dviews, want=(variant,))[0], plan)
    finally:
        del os.environ["VD_FKG_VARIANT"]
    assert {k: tuple(v[:2]) for k, v in got.items()} == exp


@pytest.mark.parametrize("variant", ["fk_select_sum_tma", "fk_select_sum_ldg", "gather_fold"])
@pytest.mark.parametrize("mode", [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED, vd.VD_SEL_PREDICATED_LOOKUP])
@pytest.mark.parametrize("sel", [0.0, 0.013, 0.5, 1.0])
def test_fkjsel_fig16_strategies_vs_interpreter(mode, sel, variant):
    """Fig 16: branching, predicated aggregation and predicated
    lookups give the same SUM(target.v) and count as the oracle's program
    Gather(target.v, fk - 1) -> FoldSelect(v < t) -> FoldSum, with epsilon in
    every column and foreign keys outside the target (gathered as epsilon)."""
    import os
    n, m = 100003, 5000
    rng = np.random.default_rng(7)
    fk = rng.integers(-1, m + 3, n).astype(np.int32)
    v = rng.integers(0, plans.FKJSEL_VMAX, n).astype(np.int32)
    tv = rng.integers(-10**6, 10**6, m).astype(np.int64)
    efk, ev, et = rng.random(n) < 0.01, rng.random(n) < 0.01, rng.random(m) < 0.01
    fk[efk], v[ev], tv[et] = -2**31, -2**31, -2**63
    thr = int(round(sel * plans.FKJSEL_VMAX))
    prog = f"""
    p := Subtract(fact.fk, 1)
    g := Gather(target.v, p)
    q := Greater({thr}, fact.v)
    pos := FoldSelect(q)
    sel := Gather(g, pos)
    s := FoldSum(sel)
    c := FoldCount(pos)
    """
    po = oracle.run(prog, fact__fk=(fk, efk), fact__v=(v, ev), target__v=(tv, et))
    exp_s, exp_c = po.get("s")[0], po.get("c")[0]
    keep, views = load([fk, v])
    dkeep, dviews = load([tv])
    plan = plans.fkjsel(thr, mode)
    fk_var = {"gather_fold": "off", "fk_select_sum_ldg": "ldg", "fk_select_sum_tma": "tma"}[variant]
    with env(VD_FKJS_VARIANT=fk_var, VD_LATE="off"):
        got = vd.decode_partials(run(plan, views, n, dviews, want=(variant.replace("_ldg", "").replace("_tma", ""),))[0],
                                 plan)
    want = {} if not exp_c else {0: [exp_s or 0, exp_c, exp_c]}
    assert got == want
    if variant == "gather_fold" and mode == vd.VD_SEL_BRANCH:
        # branching without the Fig 16 kernels: the late-materialisation fragment
        # (v < t is an i32 interval lead; fk and the lookup per qualifying row)
        with env(VD_FKJS_VARIANT="off", VD_LATE="force"):
            assert vd.decode_partials(run(plan, views, n, dviews, want=("late",))[0], plan) == want


@pytest.mark.parametrize("seed", range(10))
def test_late_fragment_random_plans_vs_oracle(seed):
    """Late-materialisation fragment on random branching plans: terms shared
    by every conjunction on two u8 columns and one i32 column (the lead
    columns: intervals, IN sets and NE that are not, epsilon in every column),
    per-conjunction terms on the other columns, a ragged row count; against
    the oracle (one FoldSelect program per conjunction, union, then Gather ->
    Multiply -> FoldSum / FoldCount)."""
    rng = np.random.default_rng(700 + seed)
    n = 50001 + 37 * seed  # n % 16 != 0: the tail rows
    cols = {"a": rng.integers(0, 40, n).astype(np.uint8), "b": rng.integers(0, 8, n).astype(np.uint8),
            "c": rng.integers(-500, 500, n).astype(np.int32), "x": rng.integers(0, 10**6, n).astype(np.int64),
            "y": rng.integers(0, 11, n).astype(np.int64), "r": rng.integers(0, 100, n).astype(np.int64)}
    eps = {}
    for k, arr in cols.items():
        m = rng.random(n) < 0.01
        arr[m] = {np.uint8: 255, np.int32: -2**31, np.int64: -2**63}[arr.dtype.type]
        eps[k] = m
    order = ["a", "b", "c", "x", "y", "r"]
    idx = {k: i for i, k in enumerate(order)}

    def term(k):
        if k in ("a", "b"):
            cmp = str(rng.choice([">", "<", ">=", "<=", "==", "!=", "in"]))
            if cmp == "in":
                lo = int(rng.integers(0, 30))
                return k, cmp, (list(range(lo, lo + int(rng.integers(1, 6)))) if rng.random() < 0.6
                                else sorted(set(int(v) for v in rng.integers(0, 40, 4))))
            return k, cmp, int(rng.integers(0, 40 if k == "a" else 8))
        if k == "c":
            return k, str(rng.choice([">", "<", ">=", "<=", "=="], p=[.3, .3, .15, .15, .1])), int(rng.integers(-400, 400))
        return k, str(rng.choice([">", "<", ">=", "<="])), int(rng.integers(0, 100))

    common = [term(k) for k in ("a", "b") if rng.random() < 0.8] + [term("c")]  # c: always an interval lead
    conjs = [common + [term("r") for _ in range(int(rng.integers(0, 3)))] for _ in range(int(rng.integers(1, 4)))]
    sel = np.zeros(n, dtype=bool)
    inputs = {f"fact__{k}": (v, eps[k]) for k, v in cols.items()}
    for terms in conjs:
        lines, names = [], []
        for j, (k, cmp, val) in enumerate(terms):
            _term_expr(f"t{j}", f"fact.{k}", cmp, val, lines)
            names.append(f"t{j}")
        lines.append(f"q := LogicalAnd({names[0]}, {names[0]})")
        for nm in names[1:]:
            lines.append(f"q := LogicalAnd(q, {nm})")
        lines.append("pos := FoldSelect(q)")
        pos, pe = oracle.run("\n".join(lines), **inputs).get_arrays("pos")
        sel[pos[~pe]] = True
    upos = np.nonzero(sel)[0].astype(np.int64)
    agg = oracle.run("""
    gx := Gather(fact.x, pos)
    gy := Gather(fact.y, pos)
    f := Multiply(gy, -1)
    t := Add(f, 100)
    pr := Multiply(gx, t)
    s := FoldSum(pr)
    c := FoldCount(pos)
    """, fact__x=(cols["x"], eps["x"]), fact__y=(cols["y"], eps["y"]), pos=upos)
    exp = {0: [int(agg.get("s")[0]), int(agg.get("c")[0]), int(agg.get("c")[0])]} if upos.size else {}
    keep, views = load([cols[k] for k in order])
    plan = vd.pipeline(pred_=vd.pred([[(idx[k], cmp, val) for k, cmp, val in t] for t in conjs]),
                       aggs=[("sum", [idx["x"], (idx["y"], 100, -1)]), ("count",)])
    with env(VD_LATE="force"):
        got = vd.decode_partials(run(plan, views, n, want=("late",))[0], plan)
    assert got == exp


def test_late_fragment_selectivity_estimate():
    """Default dispatch takes the late-materialisation fragment only when the
    lead intervals are estimated (min/max metadata, even spread) to pass few
    rows: a 2% lead on an i32 column goes late, a 60% one stays dense
    (gather-fold); VD_LATE=force takes it regardless.  Same results."""
    rng = np.random.default_rng(5)
    n, m = 200003, 5000
    fk = rng.integers(1, m + 1, n).astype(np.int32)
    v = rng.integers(0, 1000, n).astype(np.int32)
    tv = rng.integers(-10**6, 10**6, m).astype(np.int64)
    keep, views = load([fk, v])
    dkeep, dviews = load([tv])
    for thr, frag in ((20, "late"), (600, "gather_fold")):
        plan = vd.pipeline(pred_=vd.pred([[(1, "<", thr)]]), gathers=[(0, 0, 1)], aggs=[("sum", [2]), ("count",)])
        sel = v < thr
        exp = {0: [int(tv[fk[sel] - 1].sum()), int(sel.sum()), int(sel.sum())]}
        with env(VD_FKJS_VARIANT="off", VD_STAR_VARIANT="off"):
            got, _ = run(plan, views, n, dviews, want=(frag,))
            assert vd.decode_partials(got, plan) == exp
            with env(VD_LATE="force"):
                got, _ = run(plan, views, n, dviews, want=("late",))
                assert vd.decode_partials(got, plan) == exp


@pytest.mark.parametrize("late_fast", ["1", "0"])
@pytest.mark.parametrize("n", [1, 15, 16, 17, 511, 513, 4099])
@pytest.mark.parametrize("lead", ["none", "all", "some"])
def test_late_fragment_edge_sizes(n, lead, late_fast):
    """Late fragment at sizes around its 16-row lead words and 32-row drains
    (tail rows only, one word, one word + tail, partial drains) with leads
    that pass nothing, everything or some rows; against the interpreter
    (FoldSelect of the lead and the gathered dimension term, Gather,
    FoldSum / FoldCount)."""
    rng = np.random.default_rng(n * 7 + len(lead))
    m = 300
    a = rng.integers(0, 4, n).astype(np.uint8)
    fk = rng.integers(1, m + 1, n).astype(np.int32)
    x = rng.integers(-10**6, 10**6, n).astype(np.int64)
    d = rng.integers(0, 10, m).astype(np.uint8)
    cmp_, val = {"none": ("==", 9), "all": ("<=", 3), "some": ("==", 2)}[lead]
    plan = vd.pipeline(pred_=vd.pred([[(0, cmp_, val), (3, "<", 5)]]), gathers=[(1, 0, 1)],
                       aggs=[("sum", [2]), ("count",)])
    lead_term = "c1 := Equals(f.a, %d)" % val if cmp_ == "==" else "c1 := Greater(%d, f.a)" % (val + 1)
    p = oracle.Program()
    p.set("f.a", a)
    p.set("f.fk", fk)
    p.set("f.x", x)
    p.set("dim.d", d)
    p.run(lead_term + """
pk := Subtract(f.fk, 1)
dd := Gather(dim.d, pk)
c2 := Greater(5, dd)
keep := LogicalAnd(c1, c2)
positions := FoldSelect(keep)
sel := Gather(f.x, positions)
total := FoldSum(sel)
cnt := FoldCount(positions)
""")
    c = p.get("cnt")[0] if n else 0
    exp = {0: [p.get("total")[0], c, c]} if c else {}
    keep, views = load([a, fk, x])
    dkeep, dviews = load([d])
    with env(VD_LATE="force", VD_LATE_FAST=late_fast):
        got, _ = run(plan, views, n, dviews, want=("late",))
    assert vd.decode_partials(got, plan) == exp


@pytest.mark.parametrize("late_fast", ["1", "0"])
@pytest.mark.parametrize("seed", range(12))
def test_late_fragment_random_fk_plans_vs_oracle(seed, late_fast):
    """Late fragment with FK lookups on random branching plans: a common u8
    lead on the fact table, per-conjunction terms on two u8 dimension columns
    (acceptance tables: every comparison kind, IN sets, NE, codes >= 64), an
    i32 dimension column and an i64 fact column (constraints), epsilon in
    every column and FKs outside the dimension; against the oracle (one
    FoldSelect program per conjunction through Gather, union, then
    Gather -> Multiply -> FoldSum / FoldCount)."""
    rng = np.random.default_rng(900 + seed)
    n, m = 60001 + 31 * seed, 2503
    fk = rng.integers(-3, m + 5, n).astype(np.int32)
    ld = rng.integers(0, 6, n).astype(np.uint8)
    rq = rng.integers(0, 6000, n).astype(np.int64)
    x = rng.integers(0, 10**7, n).astype(np.int64)
    d1 = rng.integers(0, 80, m).astype(np.uint8)
    d2 = rng.integers(0, 40, m).astype(np.uint8)
    dr = rng.integers(1, 51, m).astype(np.int32)
    eps = {}
    for nm, arr, e in [("fk", fk, -2**31), ("ld", ld, 255), ("rq", rq, -2**63), ("x", x, -2**63),
                       ("d1", d1, 255), ("d2", d2, 255), ("dr", dr, -2**31)]:
        msk = rng.random(arr.size) < 0.01
        arr[msk] = e
        eps[nm] = msk
    ref_idx = {"fk": 0, "ld": 1, "rq": 2, "x": 3, "d1": 4, "d2": 5, "dr": 6}

    def rand_term(k):
        if k in ("d1", "d2"):
            cmp = str(rng.choice([">", "<", "==", ">=", "<=", "!=", "in"]))
            if cmp == "in":
                return k, cmp, sorted(set(int(v) for v in rng.integers(0, 64, rng.integers(1, 12))))
            return k, cmp, int(rng.integers(0, 90))
        hi = 6000 if k == "rq" else 50
        return k, str(rng.choice([">", "<", ">=", "<="])), int(rng.integers(0, hi))

    lead = ("ld", "==", int(rng.integers(0, 6)))  # ~1/6 of the rows: a selective lead
    conjs = []
    for _ in range(int(rng.integers(1, 4))):
        names = [k for k in ("d1", "d2", "dr", "rq") if rng.random() < 0.5] or ["d1"]
        conjs.append([lead] + [rand_term(k) for k in names])
    sel = np.zeros(n, dtype=bool)
    inputs = {f"fact__{k}": (v, eps[k]) for k, v in (("fk", fk), ("ld", ld), ("rq", rq))}
    inputs.update({f"dim__{k}": (v, eps[k]) for k, v in (("d1", d1), ("d2", d2), ("dr", dr))})
    oref = {"ld": "fact.ld", "rq": "fact.rq", "d1": "gd1", "d2": "gd2", "dr": "gdr"}
    for terms in conjs:
        lines = ["p := Subtract(fact.fk, 1)", "gd1 := Gather(dim.d1, p)", "gd2 := Gather(dim.d2, p)",
                 "gdr := Gather(dim.dr, p)"]
        names = []
        for j, (k, cmp, val) in enumerate(terms):
            _term_expr(f"t{j}", oref[k], cmp, val, lines)
            names.append(f"t{j}")
        lines.append(f"q := LogicalAnd({names[0]}, {names[0]})")
        for nm in names[1:]:
            lines.append(f"q := LogicalAnd(q, {nm})")
        lines.append("pos := FoldSelect(q)")
        pos, pe = oracle.run("\n".join(lines), **inputs).get_arrays("pos")
        sel[pos[~pe]] = True
    upos = np.nonzero(sel)[0].astype(np.int64)
    agg = oracle.run("""
    gx := Gather(fact.x, pos)
    s := FoldSum(gx)
    c := FoldCount(pos)
    """, fact__x=(x, eps["x"]), pos=upos)
    exp = {0: [int(agg.get("s")[0]), int(agg.get("c")[0]), int(agg.get("c")[0])]} if upos.size else {}
    keep, views = load([fk, ld, rq, x])
    dkeep, dviews = load([d1, d2, dr])
    plan = vd.pipeline(pred_=vd.pred([[(ref_idx[k], cmp, val) for k, cmp, val in t] for t in conjs]),
                       gathers=[(0, 0, 1), (0, 1, 1), (0, 2, 1)], aggs=[("sum", [3]), ("count",)])
    with env(VD_LATE="force", VD_LATE_FAST=late_fast):  # the fast first round (FK + tabulated u8 lookups) or not
        got = vd.decode_partials(run(plan, views, n, dviews, want=("late",))[0], plan)
    assert got == exp
    with env(VD_LATE="off", VD_STAR_VARIANT="off"):  # the dense gather-fold fragment agrees
        assert vd.decode_partials(run(plan, views, n, dviews, want=("gather_fold",))[0], plan) == got
