"""bench.py's algorithmic-bytes accounting for the Q19 late fragment
(DESIGN readings A31/A33/A34), checked on a hand-built table whose block
counts are known: host logic only, runs on CPU."""
import numpy as np
import torch

import bench
import gen
from paper_journals_pvldb_pirkmzm16_b200 import plans


def test_q19_late_bytes_hand_example():
    n = 64
    deliver = gen.SHIPINSTRUCT.index("DELIVER IN PERSON")
    air = gen.SHIPMODE.index("AIR")
    other_instr = (deliver + 1) % len(gen.SHIPINSTRUCT)
    other_mode = (air + 1) % len(gen.SHIPMODE)
    partkey = np.ones(n, np.int32)          # every row -> part row 0
    qty = np.full(n, 500, np.int64)        # quantity 5 (scale 100): branch 1's range
    ext = np.full(n, 1000, np.int64)
    disc = np.zeros(n, np.int64)
    mode = np.full(n, other_mode, np.uint8)
    instr = np.full(n, other_instr, np.uint8)
    # lead rows (AIR, DELIVER IN PERSON): 0, 3 and 40
    for r in (0, 3, 40):
        mode[r], instr[r] = air, deliver
    # part row 0 passes branch 1 (Brand#12, SM CASE, size 1..5), so every
    # lead row is undecided after the brand/container lookups and qualifies
    # unless its quantity is out of range: row 40 gets quantity 50
    qty[40] = 5000
    part_brand = np.array([gen.BRAND.index("Brand#12")], np.uint8)
    part_cont = np.array([gen.CONTAINER.index("SM CASE")], np.uint8)
    part_size = np.array([3], np.int32)
    cols = [torch.from_numpy(a) for a in (partkey, qty, ext, disc, mode, instr)]
    dims = [torch.from_numpy(a) for a in (part_brand, part_cont, part_size)]
    alg, extra = bench.q19_late_bytes(None, cols, dims, {0: [0, 2, 2]}, None, 1.0)
    assert extra["lead_rows"] == 3 and extra["undecided_rows"] == 3 and extra["qualifying_check"] == 2
    # leads: 2 u8 columns in full = 2n; l_partkey (i32, 16 rows per 64 B):
    # rows 0, 3 -> block 0, row 40 -> block 2; l_quantity (i64, 8 rows per
    # block) for the undecided rows 0, 3, 40 -> blocks 0 and 5; ext / disc
    # (i64) for the qualifying rows 0, 3 -> block 0 each; the part table once
    expect = 2 * n + 2 * 64 + 2 * 64 + 64 + 64 + (1 + 1 + 4)
    assert alg == expect
    assert extra["l2"]["lookups"] == 2 * 3 + 3  # brand + container per lead row, size per undecided row
    assert plans.Q19_BRANCHES[0][0] == "Brand#12"
