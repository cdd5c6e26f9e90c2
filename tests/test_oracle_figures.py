"""Pins of the oracle interpreter to the paper's worked examples and invariants.

Each test checks the oracle (layer 1) against something other than itself:
values printed in the paper's figures (tests/golden/, cited), invariants the
paper states, and closed forms.
"""
import numpy as np
import pytest

import oracle
from oracle import programs
from vd_testutil import load_golden


def test_fig7_foldsum_controlled():
    g = load_golden("fig7_foldsum.json")
    p = oracle.run("s := FoldSum(fold, value)", fold=g["fold"], value=g["value"])
    assert p.get("s") == g["sum"]


def _fig9_quantity(g, fill):
    q = np.full(len(g["v"]), fill, dtype=np.int64)
    for k, val in g["quantity_known"].items():
        q[int(k)] = val
    return q


@pytest.mark.parametrize("fill", [0, 1, 99, -7])
def test_fig9_select_gather_hierarchical_sum(fill):
    """Fig 9 through the Fig 8 program; the unseen
    l_quantity values are free, so the result must not depend on them."""
    g = load_golden("fig9_select_gather_sum.json")
    prog = programs.FIG8_SELECT_SUM.format(intent=g["intent"], threshold=g["threshold"])
    p = oracle.run(prog, lineitem__l_shipdate=g["v"], lineitem__l_quantity=_fig9_quantity(g, fill))
    assert p.get("value") == g["greater"]
    assert p.get("positions") == g["foldSelect"]
    assert p.get("q") == g["gather"]
    assert p.get("partialSum") == g["partialSum"]
    assert p.get("totalSum") == g["totalSum"]


def test_fig11_virtual_scatter_group_fold():
    g = load_golden("fig11_virtual_scatter.json")
    prog = """
    pivot := Range(0, 4, 1)
    pos := Partition(t.k, pivot)
    sc := Scatter(t, t, pos)
    s := FoldSum(sc.k, sc.v)
    c := FoldCount(sc.k, sc.v)
    gpos := FoldSelect(c)
    out := Gather(s, gpos)
    """
    p = oracle.run(prog, t__k=g["keys"], t__v=g["values"])
    assert p.get("pos") == g["partition"]
    # Scatter tags value@pos: slot pos holds value
    sv = p.get("sc.v")
    for val, pos in g["scatter_tags"]:
        assert sv[pos] == val
    assert p.get("s") == g["foldSum"]
    assert p.get("out") == g["compacted"]
    assert p.get("c") == g["foldCount_reading_A24"]


def test_fig10_program_on_fig11_data():
    """The Fig 10 plan run on the Fig 11 values gives the compacted
    sums in pivot order (reading A16)."""
    g = load_golden("fig11_virtual_scatter.json")
    prog = programs.FIG10_GROUP_SUM.format(card=4)
    p = oracle.run(prog, lineitem__l_returnflag=g["keys"], lineitem__l_quantity=g["values"])
    assert p.get("L1") == g["compacted"]
    assert p.get("K1")[:4] == [0, 1, 2, 3]
    assert p.get("C1")[:4] == [3, 3, 3, 1]


@pytest.mark.parametrize("n", [1, 7, 1023, 1024, 1025, 5000])
@pytest.mark.parametrize("seed", [1, 2])
def test_fig3_fig4_hierarchical_invariance(n, seed):
    """Fig 3 vs Fig 4: the hierarchical sum is the
    same whatever the partition size or lane count, and equals the plain sum
    (exact for integers)."""
    rng = np.random.default_rng(seed)
    x = rng.integers(-10**12, 10**12, size=n)
    plain = int(np.sum(x.astype(object)))
    for ps in [1, 3, 1024]:
        p = oracle.run(programs.FIG3_HIERARCHICAL.format(partition_size=ps), input__val=x)
        assert p.get("totalSum")[0] == plain
        # one partial per partition, each at its run start
        psum = p.get("pSum")
        nparts = (n + ps - 1) // ps
        starts = [k * ps for k in range(nparts)]
        assert [psum[s] for s in starts] == [int(np.sum(x[s:s + ps].astype(object))) for s in starts]
    for lanes in [1, 2, 4]:
        p = oracle.run(programs.FIG4_SIMD.format(lane_count=lanes), input__val=x)
        assert p.get("totalSum")[0] == plain
        psum = [v for v in p.get("pSum") if v is not None]
        assert psum == [int(np.sum(x[j::lanes].astype(object))) for j in range(min(lanes, n))]


def test_fig3_float_closed_form():
    """Sum of Range(0, n, 1) as floats = n(n-1)/2 exactly (closed form)."""
    n = 100000
    p = oracle.run(programs.FIG3_HIERARCHICAL.format(partition_size=1024),
                   input__val=np.arange(n, dtype=np.float64))
    assert p.get("totalSum")[0] == n * (n - 1) / 2


def test_fig1_branching_equals_predicated_positions():
    """Fig 1: branching and cursor-arithmetic selection are two
    implementations of one result.  The oracle's FoldSelect positions equal
    a branch-free cursor loop written in numpy and np.flatnonzero."""
    rng = np.random.default_rng(3)
    v = rng.random(5000).astype(np.float32)
    for t in [0.0, 0.01, 0.5, 0.99, 1.0]:
        t = float(np.float32(t))  # the predicate constant is an f32 (reading A20)
        # hex literal: the oracle parses the exact f32 value
        p = oracle.run("value := Greater(%s, v.val)\npos := FoldSelect(value)" % t.hex(), v__val=v)
        got = [x for x in p.get("pos") if x is not None]
        # branch-free cursor arithmetic (Ross): write every input, advance by predicate
        out = np.empty(v.size + 1, dtype=np.int64)
        cur = 0
        pred = (np.float32(t) > v).astype(np.int64)
        for i in range(v.size):
            out[cur] = i
            cur += int(pred[i])
        assert got == out[:cur].tolist() == np.flatnonzero(v < np.float32(t)).tolist()
        # brute-force layer agrees
        pos, c, _ = oracle.select_f32(v, float(np.float32(t)), "lt")
        assert c == cur and pos.tolist() == got


@pytest.mark.parametrize("chunk", [1, 32, 1000, 4096, 10**6])
def test_fig15_materialize_and_break_leave_values_unchanged(chunk):
    """Materialize / Break (Table 2) direct how a program runs,
    not what it computes: the Vectorized plan (per-chunk position lists
    materialised, chunks = runs of Divide(Range, C)) and the Break plan equal
    the fused plan and a brute-force loop over the same f32 columns (sum of
    v2 where lo <= v1 <= hi, long double vs exact rational tolerance)."""
    import numpy as np

    import gen
    from oracle import programs
    n = 20011
    v1 = gen.host(gen.F32_UNIFORM, n, seed=7)
    v2 = gen.host(gen.F32_UNIFORM, n, seed=8)
    lo, hi = np.float32(0.25), np.float32(0.6)
    m = (v1 >= lo) & (v1 <= hi)
    from fractions import Fraction
    exact = sum(Fraction(float(x)) for x in v2[m])
    # v1 >= lo <=> Greater(v1, pred(lo)); v1 <= hi <=> Greater(succ(hi), v1) on f32 values
    lom = float(np.nextafter(lo, np.float32(-1)))
    hip = float(np.nextafter(hi, np.float32(2)))
    res = []
    for prog in (programs.FIG15_FUSED, programs.FIG15_VECTORIZED, programs.FIG15_BREAK):
        p = oracle.run(prog.format(lom=lom.hex(), hip=hip.hex(), chunk=chunk), input__v1=v1, input__v2=v2)
        t, r, _ = p.get_float_exact("total")
        res.append((t[0] + r[0], p.get("count")[0]))
    for tot, cnt in res:
        assert cnt == int(m.sum())
        assert abs(Fraction(tot) - exact) <= Fraction(1, 10**9) * exact
    assert res[0] == res[2]  # Break: the same single fold order
