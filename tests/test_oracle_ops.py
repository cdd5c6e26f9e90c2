"""Pins of each oracle operator to library special cases and closed forms.

Each operator of Table 2 is checked against an independent
library routine on the special case where the two must coincide (numpy /
pandas / Python builtins), on random inputs (hypothesis), plus the
edge-case readings of SURVEY.md §8(c) that no library fixes (marked
"reading", parity unpinned by the paper).
"""
import numpy as np
import pandas as pd
import pytest
from hypothesis import given, settings
from hypothesis import strategies as st

import oracle

ints = st.lists(st.integers(-10**15, 10**15), min_size=0, max_size=60)


def _runs_by_adjacency(ctrl):
    """Run starts of a control vector via pandas: a new run where the value
    differs from its predecessor (shift/ne/cumsum idiom)."""
    s = pd.Series(ctrl)
    rid = (s != s.shift()).cumsum() - 1
    return rid.to_numpy()


@settings(max_examples=150, deadline=None)
@given(st.lists(st.tuples(st.integers(0, 3), st.integers(-1000, 1000)), min_size=1, max_size=60))
def test_foldsum_count_min_max_equal_pandas_groupby_of_runs(pairs):
    """FoldSum/Count/Min/Max = pandas groupby over
    adjacency runs, written at each run start, epsilon elsewhere."""
    ctrl = np.array([c for c, _ in pairs])
    val = np.array([v for _, v in pairs])
    p = oracle.run("""
    s := FoldSum(c, v)
    n := FoldCount(c, v)
    lo := FoldMin(c, v)
    hi := FoldMax(c, v)
    """, c=ctrl, v=val)
    rid = _runs_by_adjacency(ctrl)
    df = pd.DataFrame({"r": rid, "v": val, "i": np.arange(len(val))})
    g = df.groupby("r", sort=True).agg(s=("v", "sum"), n=("v", "size"), lo=("v", "min"), hi=("v", "max"),
                                       start=("i", "min"))
    for name in ["s", "n", "lo", "hi"]:
        exp = [None] * len(val)
        for _, row in g.iterrows():
            exp[int(row["start"])] = int(row[name])
        assert p.get(name) == exp, name


@settings(max_examples=150, deadline=None)
@given(ints)
def test_single_run_fold_is_builtin(xs):
    """One run: FoldSum = sum(), FoldMin/Max = min()/max() (library special case)."""
    if not xs:
        return
    p = oracle.run("s := FoldSum(v)\nlo := FoldMin(v)\nhi := FoldMax(v)\nn := FoldCount(v)", v=np.array(xs))
    assert p.get("s")[0] == sum(xs)
    assert p.get("lo")[0] == min(xs)
    assert p.get("hi")[0] == max(xs)
    assert p.get("n")[0] == len(xs)
    assert p.get("s")[1:] == [None] * (len(xs) - 1)


@settings(max_examples=150, deadline=None)
@given(st.lists(st.tuples(st.integers(0, 2), st.integers(0, 1)), min_size=1, max_size=60))
def test_foldselect_equals_flatnonzero_per_run(pairs):
    """FoldSelect: per run, ascending absolute positions of
    non-zero .s (np.flatnonzero), packed from the run start (Fig 9)."""
    ctrl = np.array([c for c, _ in pairs])
    s = np.array([x for _, x in pairs])
    p = oracle.run("pos := FoldSelect(c, s)", c=ctrl, s=s)
    rid = _runs_by_adjacency(ctrl)
    exp = [None] * len(s)
    for r in np.unique(rid):
        idx = np.flatnonzero(rid == r)
        sel = idx[s[idx] != 0]
        for j, pos in enumerate(sel):
            exp[idx[0] + j] = int(pos)
    assert p.get("pos") == exp


@settings(max_examples=150, deadline=None)
@given(st.lists(st.integers(0, 6), min_size=1, max_size=60), st.integers(1, 7))
def test_partition_is_stable_argsort_inverse(keys, P):
    """Partition with pivots Range(0,P,1) on keys < P is a stable
    counting sort: positions = inverse of np.argsort(kind='stable')."""
    keys = [k % P for k in keys]
    p = oracle.run("piv := Range(0, %d, 1)\npos := Partition(k, piv)" % P, k=np.array(keys))
    order = np.argsort(np.array(keys), kind="stable")
    inv = np.empty(len(keys), dtype=np.int64)
    inv[order] = np.arange(len(keys))
    assert p.get("pos") == inv.tolist()


def test_partition_pivot_buckets_reading_A13():
    """Reading A13: bucket = upper_bound(pivots, v) - 1, clamped at 0 (np.searchsorted)."""
    v = np.array([5, -3, 17, 10, 10, 0, 25, 9])
    piv = np.array([0, 10, 20])
    p = oracle.run("pos := Partition(v, piv)", v=v, piv=piv)
    b = np.clip(np.searchsorted(piv, v, side="right") - 1, 0, None)
    inv = np.empty(len(v), dtype=np.int64)
    inv[np.argsort(b, kind="stable")] = np.arange(len(v))
    assert p.get("pos") == inv.tolist()


@settings(max_examples=150, deadline=None)
@given(st.lists(st.integers(-1000, 1000), min_size=1, max_size=40),
       st.lists(st.integers(-5, 45), min_size=0, max_size=40))
def test_gather_is_fancy_indexing_with_oob_epsilon(src, pos):
    """Gather: out size |pos|; out = src[pos], OOB -> epsilon (A11)."""
    p = oracle.run("g := Gather(s, p)", s=np.array(src), p=np.array(pos, dtype=np.int64))
    exp = [src[q] if 0 <= q < len(src) else None for q in pos]
    if not pos:
        exp = []
    assert p.get("g") == exp


@settings(max_examples=150, deadline=None)
@given(st.lists(st.tuples(st.integers(-1000, 1000), st.integers(-3, 20)), min_size=1, max_size=40),
       st.integers(1, 20))
def test_scatter_last_writer_wins_like_dict(pairs, out_len):
    """Scatter: slots not written are epsilon; in input order, so
    a later write overwrites (reading A12) -- a Python dict built in input
    order is the same mapping.  OOB positions are dropped."""
    vals = np.array([v for v, _ in pairs])
    pos = np.array([q for _, q in pairs])
    p = oracle.run("o := Scatter(v, %d, p)" % out_len, v=vals, p=pos)
    d = {}
    for v, q in pairs:
        if 0 <= q < out_len:
            d[q] = v
    assert p.get("o") == [d.get(k) for k in range(out_len)]


def test_scatter_of_permutation_inverts_gather():
    """For a permutation, Scatter by pi then Gather by pi is the identity."""
    rng = np.random.default_rng(5)
    x = rng.integers(-10**9, 10**9, size=500)
    pi = rng.permutation(500)
    p = oracle.run("s := Scatter(x, x, pi)\ng := Gather(s, pi)", x=x, pi=pi)
    assert p.get("g") == x.tolist()
    assert p.get("s") == x[np.argsort(pi)].tolist()


@pytest.mark.parametrize("n,R", [(1, 1), (10, 1), (10, 3), (4096, 1024), (1000, 7)])
def test_virtual_ctrl_equals_divide_and_modulo_reading_A2(n, R):
    """Run metadata (reading A2): Ctrl(0,1,R,0) == Divide(Range, R)
    ('dividing by x divides step by x') and Ctrl(0,1,1,R) == Modulo(Range, R)
    ('a modulo by x sets cap to x')."""
    p = oracle.run(f"""
    ids := Range(0, {n}, 1)
    d := Divide(ids, {R})
    m := Modulo(ids, {R})
    vd := Ctrl(0, 1, {R}, 0, {n})
    vm := Ctrl(0, 1, 1, {R}, {n})
    dm := Ctrl(0, 1, {R}, 2, {n})
    dm2 := Modulo(d, 2)
    """)
    assert p.get("vd") == p.get("d") == (np.arange(n) // R).tolist()
    assert p.get("vm") == p.get("m") == (np.arange(n) % R).tolist()
    assert p.get("dm") == p.get("dm2")


def test_runs_are_adjacent_blocks_reading_A3():
    """Reading A3: non-contiguous repeats are separate runs."""
    p = oracle.run("s := FoldSum(c, v)", c=[0, 0, 1, 1, 0, 0], v=[1, 2, 3, 4, 5, 6])
    assert p.get("s") == [3, None, 7, None, 11, None]


def test_epsilon_rules_reading_A5_A9():
    """Reading A5/A9 (parity unpinned by the paper): epsilon is skipped by
    folds, an all-epsilon run sums/counts to 0 and has epsilon min/max, and
    epsilon propagates through arithmetic and comparisons."""
    v = np.array([4, 7, 1, 2, 9, 3])
    eps = [1, 1, 0, 1, 0, 0]
    p = oracle.run("""
    s := FoldSum(c, v)
    n := FoldCount(c, v)
    lo := FoldMin(c, v)
    a := Add(v, 1)
    g := Greater(v, 2)
    """, c=[0, 0, 1, 1, 2, 2], v=(v, eps))
    assert p.get("s") == [0, None, 1, None, 12, None]
    assert p.get("n") == [0, None, 1, None, 2, None]
    assert p.get("lo") == [None, None, 1, None, 3, None]
    assert p.get("a") == [None, None, 2, None, 10, 4]
    assert p.get("g") == [None, None, 0, None, 1, 1]


def test_arithmetic_shorter_length_and_c_division():
    """output size is the smaller input; Divide/Modulo truncate (A10)."""
    p = oracle.run("d := Divide(a, b)\nm := Modulo(a, b)", a=[7, -7, 9, 100], b=[2, 2, -4])
    assert p.get("d") == [3, -3, -2]
    assert p.get("m") == [1, -1, 1]


def test_int128_sums_do_not_wrap():
    """Q1's sum_charge exceeds int64 at SF100 (reading A17): 128-bit sums."""
    big = np.full(4, 2**62, dtype=np.int64)
    p = oracle.run("s := FoldSum(v)", v=big)
    assert p.get("s")[0] == 2**64


def test_foldscan_inclusive_restart_reading_A27():
    """FoldScan: prefix sum restarting at each run; reading A27
    (inclusive) equals np.cumsum per run."""
    c = np.array([0, 0, 0, 1, 1, 2])
    v = np.array([1, 2, 3, 4, 5, 6])
    p = oracle.run("s := FoldScan(c, v)", c=c, v=v)
    assert p.get("s") == [1, 3, 6, 4, 9, 6]


@settings(max_examples=150, deadline=None)
@given(st.lists(st.tuples(st.integers(-2**40, 2**40), st.integers(-20, 20)), min_size=1, max_size=40))
def test_bitshift_equals_numpy_shifts(pairs):
    """BitShift (Table 2 arithmetic): x << k for k >= 0, arithmetic
    x >> -k for k < 0 -- numpy's left_shift / right_shift on int64 (the
    operands are small enough that no bit leaves 64 bits)."""
    x = np.array([a for a, _ in pairs], dtype=np.int64)
    k = np.array([b for _, b in pairs], dtype=np.int64)
    p = oracle.run("s := BitShift(x, k)", x=x, k=k)
    exp = np.where(k >= 0, np.left_shift(x, np.maximum(k, 0)), np.right_shift(x, np.maximum(-k, 0)))
    assert p.get("s") == exp.tolist()
    # the BitShift by a constant of the Fig 3 / A15 composite key: x*2^b
    p = oracle.run("s := BitShift(x, 3)", x=x)
    assert p.get("s") == (x * 8).tolist()


@settings(max_examples=150, deadline=None)
@given(st.lists(st.tuples(st.integers(0, 3), st.integers(-1000, 1000), st.booleans()), min_size=1, max_size=60))
def test_foldscan_equals_pandas_cumsum_of_runs_with_epsilon(triples):
    """FoldScan (reading A27): per adjacency run, the inclusive
    cumulative sum of the non-epsilon values (pandas groupby.cumsum over the
    runs with epsilon as 0); an epsilon slot stays epsilon."""
    ctrl = np.array([c for c, _, _ in triples])
    val = np.array([v for _, v, _ in triples])
    eps = np.array([e for _, _, e in triples])
    p = oracle.run("s := FoldScan(c, v)", c=ctrl, v=(val, eps))
    rid = _runs_by_adjacency(ctrl)
    cs = pd.Series(np.where(eps, 0, val)).groupby(rid).cumsum().to_numpy()
    exp = [None if e else int(x) for x, e in zip(cs, eps)]
    assert p.get("s") == exp
