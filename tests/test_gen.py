"""The shared input generator: partition invariance, ranges and the
dbgen-derived shape statistics of SURVEY.md §8(d) (pin P9)."""
import numpy as np
import pytest

import gen


def test_partition_invariance_and_threads():
    sf = 0.01
    n = gen.lineitem_rows(sf)
    for name, col in gen.LINEITEM_COLS.items():
        whole = gen.host(col, n, sf=sf)
        parts = np.concatenate([gen.host(col, b - a, a, sf=sf) for a, b in [(0, 7), (7, 1000), (1000, n)]])
        assert np.array_equal(whole, parts), name
        assert np.array_equal(whole, gen.host(col, n, sf=sf, threads=4)), name


def test_ranges_and_dtypes():
    sf = 0.01
    n = gen.lineitem_rows(sf)
    li = {k: gen.host(c, n, sf=sf) for k, c in gen.LINEITEM_COLS.items()}
    assert li["l_shipdate"].dtype == np.int32 and li["l_quantity"].dtype == np.int64
    assert li["l_returnflag"].dtype == np.uint8
    assert 8036 <= li["l_shipdate"].min() and li["l_shipdate"].max() <= 10561
    assert set(np.unique(li["l_returnflag"])) <= {0, 1, 2}
    assert set(np.unique(li["l_linestatus"])) == {0, 1}
    assert li["l_quantity"].min() == 100 and li["l_quantity"].max() == 5000
    assert li["l_discount"].min() == 0 and li["l_discount"].max() == 10
    assert li["l_tax"].min() == 0 and li["l_tax"].max() == 8
    assert li["l_partkey"].min() >= 1 and li["l_partkey"].max() <= gen.part_rows(sf)
    assert li["l_suppkey"].min() >= 1 and li["l_suppkey"].max() <= gen.supplier_rows(sf)
    # extendedprice = qty * retail(partkey) (TPC-H 4.2.3) and < 2^24 (narrow products)
    pk = li["l_partkey"].astype(np.int64)
    retail = 90000 + ((pk // 10) % 20001) + 100 * (pk % 1000)
    assert np.array_equal(li["l_extendedprice"], (li["l_quantity"] // 100) * retail)
    assert li["l_extendedprice"].max() < 2**24
    # returnflag/linestatus consistent with dbgen's rule: R/A only when shipped before current date
    assert np.all(li["l_linestatus"][li["l_returnflag"] != 1] == 0)


def test_q1_q6_shape_statistics():
    """SURVEY §8(d) derived shape: Q1 keeps 98.59%; (A,F)~(R,F)~24.7%,
    (N,F) 0.64%, (N,O) 48.6% of all rows; Q6 selectivity 1.90%."""
    sf = 0.1
    n = gen.lineitem_rows(sf)
    ship = gen.host(gen.L_SHIPDATE, n, sf=sf, threads=8)
    rf = gen.host(gen.L_RETURNFLAG, n, sf=sf, threads=8)
    ls = gen.host(gen.L_LINESTATUS, n, sf=sf, threads=8)
    disc = gen.host(gen.L_DISCOUNT, n, sf=sf, threads=8)
    qty = gen.host(gen.L_QUANTITY, n, sf=sf, threads=8)
    keep = ship <= 10471
    assert keep.mean() == pytest.approx(0.98594, abs=0.002)
    k = rf.astype(int) * 2 + ls
    frac = {g: ((k == g) & keep).mean() for g in range(6)}
    assert frac[0] == pytest.approx(0.2468, abs=0.004)
    assert frac[4] == pytest.approx(0.2468, abs=0.004)
    assert frac[2] == pytest.approx(0.0064, abs=0.0015)
    assert frac[3] == pytest.approx(0.4859, abs=0.004)
    assert frac[1] == 0 and frac[5] == 0
    q6 = (ship >= 8766) & (ship < 9131) & (disc >= 5) & (disc <= 7) & (qty < 2400)
    assert q6.mean() == pytest.approx(0.01903, abs=0.0008)


def test_float_column_and_permutation():
    v = gen.host(gen.F32_UNIFORM, 1 << 16)
    assert v.dtype == np.float32 and v.min() >= 0 and v.max() < 1
    assert abs(float((v < 0.5).mean()) - 0.5) < 0.01
    # every value is a multiple of 2^-24 (exact f32)
    assert np.all((v.astype(np.float64) * 2**24) % 1 == 0)
    for n in [1, 2, 3, 1000, 65537]:
        pi = gen.host(gen.I32_PERM, n, p0=n)
        assert np.array_equal(np.sort(pi), np.arange(n))
    u = gen.host(gen.I32_UNIFORM, 10000, p0=-5, p1=9)
    assert u.min() == -5 and u.max() == 9
