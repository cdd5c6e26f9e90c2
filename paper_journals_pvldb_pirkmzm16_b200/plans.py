"""vd_pipeline descriptors of the hot-path workloads (BASELINE.json configs).

The plans are the Voodoo fragments a frontend would emit for these queries
(§4: predication / parallelisation flags, identity hashing on
min/max-sized domains); the constants are TPC-H's [ext: TPC-H spec] as
restated in SURVEY.md §8(c) reading A18, on the fixed-point layout of
DESIGN.md (DECIMAL(15,2) -> int64 x 10^2, DATE -> int32 days since
1970-01-01, CHAR -> uint8 order-preserving dictionary codes).
"""
from __future__ import annotations

from .vd import VD_SEL_BRANCH, pipeline, pred

# Column orders expected by each plan
Q1_COLS = ["l_shipdate", "l_returnflag", "l_linestatus", "l_quantity", "l_extendedprice", "l_discount", "l_tax"]
Q6_COLS = ["l_shipdate", "l_discount", "l_quantity", "l_extendedprice"]
Q19_COLS = ["l_partkey", "l_quantity", "l_extendedprice", "l_discount", "l_shipmode", "l_shipinstruct"]
Q19_DIMS = ["p_brand", "p_container", "p_size"]
Q9_COLS = ["l_suppkey", "l_shipdate", "l_extendedprice", "l_discount"]
Q9_DIMS = ["s_nationkey"]

Q1_SHIP_MAX = 10471  # 1998-12-01 - 90 days = 1998-09-02


def q1(sel_mode=VD_SEL_BRANCH, ship_max=Q1_SHIP_MAX, force_generic=False):
    """TPC-H Q1: filter + grouped aggregation over (returnflag, linestatus).

    Group key rf*2 + ls over the dictionary codes (A=0,N=1,R=2; F=0,O=1): the
    parallel grouped aggregation of P:L951-956 with a 6-slot identity-hashed
    domain.  Aggregates (scales 10^2, 10^2, 10^4, 10^6, 10^2):
    sum_qty, sum_base_price, sum_disc_price = sum(ext*(100-disc)),
    sum_charge = sum(ext*(100-disc)*(100+tax)), sum_disc, count_order."""
    return pipeline(
        pred_=pred([[(0, "<=", ship_max)]]), sel_mode=sel_mode,
        key=[(1, 0, 0, 2), (2, 0, 0, 1)], ngroups=6,
        aggs=[("sum", [3]), ("sum", [4]), ("sum", [4, (5, 100, -1)]), ("sum", [4, (5, 100, -1), (6, 100, 1)]),
              ("sum", [5]), ("count",)],
        force_generic=force_generic)


def q6(sel_mode=VD_SEL_BRANCH, d0=8766, d1=9131, dlo=5, dhi=7, qmax=2400, force_generic=False):
    """TPC-H Q6: sum(l_extendedprice * l_discount) over shipdate in [d0, d1),
    discount in [dlo, dhi], quantity < qmax (the Fig 8 plan shape)."""
    return pipeline(
        pred_=pred([[(0, ">=", d0), (0, "<", d1), (1, ">=", dlo), (1, "<=", dhi), (2, "<", qmax)]]),
        sel_mode=sel_mode, aggs=[("sum", [3, 1]), ("count",)], force_generic=force_generic)


def selsum(t: float, sel_mode=VD_SEL_BRANCH, force_generic=False):
    """Selective aggregation (Fig 15, C1): select v < t, FoldSum(v) in f64 + count."""
    return pipeline(pred_=pred([[(0, "<", float(t))]]), sel_mode=sel_mode, aggs=[("sum", [0]), ("count",)],
                    force_generic=force_generic)


def selagg(lo: float, hi: float, sel_mode=VD_SEL_BRANCH, materialize=0, mat_chunk=0):
    """Fig 15's selective aggregation:
    SELECT sum(v2) FROM t WHERE v1 BETWEEN lo AND hi, over columns [v1, v2]
    (f32, f64 accumulation) + count.  materialize / mat_chunk pick the plan:
    fused (branching / predicated), Break, or the Vectorized plan's
    Materialize of per-chunk position lists."""
    return pipeline(pred_=pred([[(0, ">=", float(lo)), (0, "<=", float(hi))]]), sel_mode=sel_mode,
                    aggs=[("sum", [1]), ("count",)], materialize=materialize, mat_chunk=mat_chunk)


# the three branches of TPC-H Q19: brand, containers, quantity lower bound
# (the upper is +10), maximum p_size
Q19_BRANCHES = [("Brand#12", ["SM CASE", "SM BOX", "SM PACK", "SM PKG"], 1, 5),
                ("Brand#23", ["MED BAG", "MED BOX", "MED PKG", "MED PACK"], 10, 10),
                ("Brand#34", ["LG CASE", "LG BOX", "LG PACK", "LG PKG"], 20, 15)]


def q19(codes, sel_mode=VD_SEL_BRANCH, force_generic=False):
    """Q19-style FK gather join (C5): lineitem x part through l_partkey - 1,
    the three-branch disjunctive predicate of TPC-H Q19, sum(ext*(100-disc)).
    `codes` maps dictionary strings to codes: {'brand': {...}, 'container':
    {...}, 'shipmode': {...}, 'shipinstruct': {...}}."""
    B, C, M, I_ = codes["brand"], codes["container"], codes["shipmode"], codes["shipinstruct"]
    modes = [M[m] for m in ("AIR", "AIR REG") if m in M]  # 'AIR REG' is not a dbgen value (A26)
    conjs = []
    for brand, conts, qlo, smax in Q19_BRANCHES:
        conjs.append([(6, "==", B[brand]), (7, "in", [C[c] for c in conts]), (1, ">=", qlo * 100),
                      (1, "<=", (qlo + 10) * 100), (8, ">=", 1), (8, "<=", smax), (4, "in", modes),
                      (5, "==", I_["DELIVER IN PERSON"])])
    return pipeline(pred_=pred(conjs), sel_mode=sel_mode, gathers=[(0, 0, 1), (0, 1, 1), (0, 2, 1)],
                    aggs=[("sum", [2, (3, 100, -1)]), ("count",)], force_generic=force_generic)


def q9(sel_mode=VD_SEL_BRANCH, force_generic=False):
    """Q9-style FK gather + grouped fold (C5): nation via l_suppkey - 1, group
    nation*7 + (year(l_shipdate) - 1992) (175 groups), sum(ext*(100-disc)), count."""
    return pipeline(sel_mode=sel_mode, gathers=[(0, 0, 1)], key=[(4, 0, 0, 7), (1, 1, 1992, 1)], ngroups=175,
                    aggs=[("sum", [2, (3, 100, -1)]), ("count",)], force_generic=force_generic)


# Fig 16 selective FK join: a 1 GiB target (128 Mi int64 rows), far larger than the 126 MB L2
# (a 128 MB target is about L2-sized: its lookups hit L2 and overstate the HBM fraction)
FKJSEL_TARGET_ROWS = 128 * 1024 * 1024
FKJSEL_VMAX = 1_000_000


def fkjsel(threshold: int, sel_mode=VD_SEL_BRANCH, force_generic=False):
    """Selective FK join (Fig 16): SELECT sum(target.v) FROM
    fact, target WHERE fact.fk = target.pk AND fact.v < threshold.  Columns:
    fact [fk (int32, 1-based), v (int32)], dims [target.v (int64)].  The
    three strategies of Fig 16 are sel_mode BRANCH / PREDICATED (predicated
    aggregation) / PREDICATED_LOOKUP (position x predicate)."""
    return pipeline(pred_=pred([[(1, "<", int(threshold))]]), sel_mode=sel_mode, gathers=[(0, 0, 1)],
                    aggs=[("sum", [2]), ("count",)], force_generic=force_generic)
