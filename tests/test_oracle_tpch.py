"""The oracle's two layers pin each other on the TPC-H-shaped workloads.

Layer 1 (interpreter running the Voodoo programs of oracle/programs.py) vs
layer 2 (brute-force C loops) vs pandas / numpy (library) on generated
tables.  Exact integer equality everywhere.
"""
import datetime

import numpy as np
import pandas as pd
import pytest

import gen
import oracle
from oracle import programs


def lineitem(sf, seed=gen.DEFAULT_SEED):
    n = gen.lineitem_rows(sf)
    return {k: gen.host(c, n, sf=sf, seed=seed) for k, c in gen.LINEITEM_COLS.items()}


def bind(p, prefix, cols):
    for k, v in cols.items():
        p.set(f"{prefix}.{k}", v)


def pandas_q1(li, ship_max=10471):
    df = pd.DataFrame({k: li[k].astype(object) if li[k].dtype == np.int64 else li[k] for k in li})
    df = df[li["l_shipdate"] <= ship_max].copy()
    df["k"] = df["l_returnflag"].astype(int) * 2 + df["l_linestatus"].astype(int)
    df["dp"] = df["l_extendedprice"] * (100 - df["l_discount"])
    df["ch"] = df["dp"] * (100 + df["l_tax"])
    g = df.groupby("k").agg(q=("l_quantity", "sum"), b=("l_extendedprice", "sum"), dp=("dp", "sum"),
                            ch=("ch", "sum"), d=("l_discount", "sum"), c=("l_quantity", "size"))
    return {int(k): [int(x) for x in row] for k, row in zip(g.index, g.to_numpy())}


@pytest.mark.parametrize("sf", [0.0002, 0.002])
def test_q1_interpreter_bruteforce_pandas(sf):
    li = lineitem(sf)
    bf = oracle.q1(li)
    assert bf == pandas_q1(li)
    p = oracle.Program()
    bind(p, "lineitem", li)
    p.run(programs.Q1.format(ship_max_p1=10472))
    keys = [k for k in p.get("o_key") if k is not None]
    got = {k: [p.get(o)[j] for o in programs.Q1_OUTPUTS] for j, k in enumerate(keys)}
    assert got == bf
    assert keys == sorted(keys)  # ascending key order (reading A16)


def test_q1_sharded_merge_equals_whole():
    """Pin P8: row-range shards (the Fig 3 ctrl one level up)
    merged by addition equal the whole-table result."""
    sf = 0.002
    li = lineitem(sf)
    n = len(li["l_shipdate"])
    whole = oracle.q1(li)
    for G in [2, 3, 8]:
        acc = {}
        for r in range(G):
            a, b = r * n // G, (r + 1) * n // G
            part = oracle.q1({k: v[a:b] for k, v in li.items()})
            for k, vals in part.items():
                acc[k] = [x + y for x, y in zip(acc.get(k, [0] * 6), vals)]
        assert acc == whole


@pytest.mark.parametrize("intent", [1, 4, 1024, 10**9])
def test_q6_interpreter_bruteforce_numpy(intent):
    li = lineitem(0.002)
    rev, cnt = oracle.q6(li)
    m = ((li["l_shipdate"] >= 8766) & (li["l_shipdate"] < 9131) & (li["l_discount"] >= 5)
         & (li["l_discount"] <= 7) & (li["l_quantity"] < 2400))
    assert cnt == int(m.sum())
    assert rev == int(np.sum(li["l_extendedprice"][m].astype(object) * li["l_discount"][m].astype(object)))
    p = oracle.Program()
    bind(p, "lineitem", li)
    p.run(programs.Q6.format(intent=intent, d0m1=8765, d1=9131, dlom1=4, dhip1=8, qmax=2400))
    assert p.get("revenue")[0] == rev
    assert p.get("count")[0] == cnt


@pytest.mark.parametrize("intent", [1, 32, 4096, 10**9])
def test_select_sum_interpreter_bruteforce(intent):
    n = 20000
    v = gen.host(gen.F32_UNIFORM, n)
    t = float(np.float32(0.5))
    pos, c, (sh, sl) = oracle.select_f32(v, t, "lt")
    assert pos.tolist() == np.flatnonzero(v < np.float32(t)).tolist()
    p = oracle.Program()
    p.set("input.val", v)
    p.run(programs.SELECT_SUM.format(intent=intent, t=t.hex()))
    assert p.get("count")[0] == c
    got = p.get_float_exact("totalSum")
    assert got[0][0] + got[1][0] == pytest.approx(sh + sl, rel=1e-15)
    assert np.isclose(sh, np.sum(v[v < np.float32(t)], dtype=np.float64), rtol=1e-12)
    sel = [x for x in p.get("positions") if x is not None]
    assert sel == pos.tolist()  # runs concatenate to the global list


def _dims(sf, seed=gen.DEFAULT_SEED):
    npart, nsupp = gen.part_rows(sf), gen.supplier_rows(sf)
    part = {k: gen.host(c, npart, sf=sf, seed=seed) for k, c in gen.PART_COLS.items()}
    supp = {k: gen.host(c, nsupp, sf=sf, seed=seed) for k, c in gen.SUPPLIER_COLS.items()}
    return part, supp


def test_year_of_day_is_datetime():
    for d in [0, 8035, 8400, 9131, 10561, 11000, 365, 730, 1095, 1461]:
        assert oracle.year_of_day(d) == (datetime.date(1970, 1, 1) + datetime.timedelta(days=d)).year


def test_fkj_q9_interpreter_bruteforce_pandas():
    sf = 0.002
    li = lineitem(sf)
    part, supp = _dims(sf)
    bf = oracle.fkj(1, li, part, supp)
    # pandas: merge on dense FK positions, group by nation*7 + year-1992
    df = pd.DataFrame({"s": li["l_suppkey"] - 1, "ship": li["l_shipdate"],
                       "rev": li["l_extendedprice"].astype(object) * (100 - li["l_discount"]).astype(object)})
    df["nat"] = supp["s_nationkey"][df["s"].to_numpy()].astype(int)
    df["yr"] = [(datetime.date(1970, 1, 1) + datetime.timedelta(days=int(d))).year for d in df["ship"]]
    df["g"] = df["nat"] * 7 + df["yr"] - 1992
    g = df.groupby("g").agg(r=("rev", "sum"), c=("rev", "size"))
    assert bf == {int(k): (int(r), int(c)) for k, (r, c) in zip(g.index, g.to_numpy())}
    # interpreter with a calendar dimension (positional date -> year lookup)
    day0 = 8000
    cal = np.array([(datetime.date(1970, 1, 1) + datetime.timedelta(days=day0 + i)).year for i in range(3000)])
    p = oracle.Program()
    bind(p, "lineitem", li)
    p.set("supplier.s_nationkey", supp["s_nationkey"])
    p.set("calendar.year", cal)
    p.run(programs.FKJ_Q9.format(day0=day0))
    keys = [k for k in p.get("o_key") if k is not None]
    got = {k: (p.get("o_rev")[j], p.get("o_cnt")[j]) for j, k in enumerate(keys)}
    assert got == bf


def test_fkj_q19_bruteforce_pandas():
    sf = 0.01
    li = lineitem(sf)
    part, supp = _dims(sf)
    bf = oracle.fkj(0, li, part, supp)
    p = li["l_partkey"] - 1
    brand = part["p_brand"][p]
    cont = part["p_container"][p]
    size = part["p_size"][p]
    C = {s: i for i, s in enumerate(gen.CONTAINER)}
    B = {s: i for i, s in enumerate(gen.BRAND)}
    M = {s: i for i, s in enumerate(gen.SHIPMODE)}
    I_ = {s: i for i, s in enumerate(gen.SHIPINSTRUCT)}
    mode_ok = np.isin(li["l_shipmode"], [M[m] for m in ["AIR", "AIR REG"] if m in M])
    instr_ok = li["l_shipinstruct"] == I_["DELIVER IN PERSON"]
    q = li["l_quantity"]
    m = np.zeros(len(q), dtype=bool)
    for b, conts, qlo, smax in [("Brand#12", ["SM CASE", "SM BOX", "SM PACK", "SM PKG"], 1, 5),
                                ("Brand#23", ["MED BAG", "MED BOX", "MED PKG", "MED PACK"], 10, 10),
                                ("Brand#34", ["LG CASE", "LG BOX", "LG PACK", "LG PKG"], 20, 15)]:
        m |= ((brand == B[b]) & np.isin(cont, [C[c] for c in conts]) & (q >= qlo * 100) & (q <= (qlo + 10) * 100)
              & (size >= 1) & (size <= smax) & mode_ok & instr_ok)
    rev = int(np.sum(li["l_extendedprice"][m].astype(object) * (100 - li["l_discount"][m]).astype(object)))
    exp = {0: (rev, int(m.sum()))} if m.sum() else {}
    assert bf == exp
    assert m.sum() > 0  # the workload selects something at this size


@pytest.mark.parametrize("sf", [0.002, 0.01])
def test_q15_interpreter_bruteforce_pandas(sf):
    """NEXT-4 pin: the Q15 revenue view grouped by l_suppkey (a large key
    domain: every supplier is a group).  Brute force (sort + runs) ==
    pandas groupby == the interpreter's Fig 10/11 program whose pivots
    cover the key's min..max range."""
    li = lineitem(sf)
    d0, d1 = 9496, 9587
    bf = oracle.q15(li, d0, d1)
    m = (li["l_shipdate"] >= d0) & (li["l_shipdate"] < d1)
    df = pd.DataFrame({"k": li["l_suppkey"][m],
                       "rev": li["l_extendedprice"][m].astype(object) * (100 - li["l_discount"][m]).astype(object)})
    g = df.groupby("k").agg(r=("rev", "sum"), c=("rev", "size"))
    assert bf == {int(k): (int(r), int(c)) for k, (r, c) in zip(g.index, g.to_numpy())}
    assert len(bf) > 0.5 * gen.supplier_rows(sf)  # high cardinality: most suppliers are groups
    kmin, kmax = int(li["l_suppkey"].min()), int(li["l_suppkey"].max())
    p = oracle.Program()
    bind(p, "lineitem", li)
    p.run(programs.Q15.format(d0m1=d0 - 1, d1=d1, kmin=kmin, D=kmax - kmin + 1))
    keys = [k for k in p.get("o_key") if k is not None]
    got = {k + kmin: (p.get("o_rev")[j], p.get("o_cnt")[j]) for j, k in enumerate(keys)}
    assert got == bf


def _q1_with_eps_bruteforce(li, eps, ship_max=10471):
    """Q1 over epsilon-laden rows by plain Python loops, from the rules
    alone: a term over epsilon is false (A9), an epsilon key code gives the
    row no group, an epsilon operand makes a product epsilon and a SUM skips
    epsilon values (A5); COUNT(*) counts the group's rows."""
    acc = {}
    n = len(li["l_shipdate"])
    for i in range(n):
        if eps["l_shipdate"][i] or not li["l_shipdate"][i] <= ship_max:
            continue
        if eps["l_returnflag"][i] or eps["l_linestatus"][i]:
            continue
        k = int(li["l_returnflag"][i]) * 2 + int(li["l_linestatus"][i])
        a = acc.setdefault(k, [0] * 6)
        q, e, d, t = (None if eps[c][i] else int(li[c][i]) for c in ("l_quantity", "l_extendedprice",
                                                                     "l_discount", "l_tax"))
        if q is not None:
            a[0] += q
        if e is not None:
            a[1] += e
        if e is not None and d is not None:
            a[2] += e * (100 - d)
            if t is not None:
                a[3] += e * (100 - d) * (100 + t)
        if d is not None:
            a[4] += d
        a[5] += 1
    return acc


@pytest.mark.parametrize("frac", [0.0, 0.05, 0.5])
def test_q1_program_with_epsilon_equals_rule_loop(frac):
    """Pins the interpreter's Q1 program (programs.Q1 + COUNT(*) = FoldCount
    over the scattered key) on epsilon-laden input -- the expected values the
    GPU epsilon tests take from it -- against a loop over the A5/A9 rules."""
    n = 3000
    li = {k: gen.host(c, n, sf=0.01) for k, c in gen.LINEITEM_COLS.items()}
    rng = np.random.default_rng(int(frac * 100) + 1)
    cols = ["l_shipdate", "l_returnflag", "l_linestatus", "l_quantity", "l_extendedprice", "l_discount", "l_tax"]
    eps = {c: rng.random(n) < frac for c in cols}
    p = oracle.Program()
    for c in cols:
        p.set("lineitem." + c, li[c], eps[c])
    p.run(programs.Q1.format(ship_max_p1=10472) + """
rows := FoldCount(sc.key, sc.key)
gpos2 := FoldSelect(rows)
r_key := Gather(gkey, gpos2)
r_qty := Gather(s_qty, gpos2)
r_base := Gather(s_base, gpos2)
r_dp := Gather(s_dp, gpos2)
r_ch := Gather(s_ch, gpos2)
r_disc := Gather(s_disc, gpos2)
r_rows := Gather(rows, gpos2)
""")
    outs = [p.get(o) for o in ("r_qty", "r_base", "r_dp", "r_ch", "r_disc", "r_rows")]
    got = {k: [(o[j] or 0) for o in outs] for j, k in enumerate(p.get("r_key")) if k is not None}
    assert got == _q1_with_eps_bruteforce(li, eps)
    if frac == 0.0:
        assert got == oracle.q1(li)


@pytest.mark.parametrize("frac", [0.0, 0.05, 0.5])
def test_q6_program_with_epsilon_equals_rule_loop(frac):
    """The same pin for programs.Q6 with COUNT(*) = FoldSum of FoldCount(fold,
    positions): a row qualifies only if every term is non-epsilon and true;
    an epsilon l_extendedprice makes the product epsilon (skipped)."""
    n = 5000
    li = {k: gen.host(c, n, sf=0.01) for k, c in gen.LINEITEM_COLS.items()}
    # widen the window so that many rows qualify
    rng = np.random.default_rng(int(frac * 100) + 2)
    cols = ["l_shipdate", "l_discount", "l_quantity", "l_extendedprice"]
    eps = {c: rng.random(n) < frac for c in cols}
    p = oracle.Program()
    for c in cols:
        p.set("lineitem." + c, li[c], eps[c])
    p.run(programs.Q6.format(intent=97, d0m1=8000, d1=10000, dlom1=2, dhip1=9, qmax=4000)
          + "pc2 := FoldCount(fold, positions)\ncount2 := FoldSum(pc2)\n")
    rev = cnt = 0
    for i in range(n):
        if any(eps[c][i] for c in ("l_shipdate", "l_discount", "l_quantity")):
            continue
        if 8001 <= li["l_shipdate"][i] < 10000 and 3 <= li["l_discount"][i] <= 8 and li["l_quantity"][i] < 4000:
            cnt += 1
            if not eps["l_extendedprice"][i]:
                rev += int(li["l_extendedprice"][i]) * int(li["l_discount"][i])
    assert (p.get("revenue")[0] or 0, p.get("count2")[0]) == (rev, cnt)
