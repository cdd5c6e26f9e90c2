"""The N>1 path's host logic on CPU: world_size-2 gloo process group.

Each rank takes its row range (dist.shard_range), produces its partials in
the vd_partials layout, and the ranks exchange and merge them
(dist.exchange_and_merge: all-gather + vd_merge_partials, which also
compacts: empty groups dropped, ascending key).  With no GPU on
this machine the per-rank partials come from the oracle's brute-force Q1 on
the rank's shard (packed into the ABI layout); the merged result must equal
the whole-table oracle (pin P8)."""
import os
import socket
import struct

import pytest
import torch.multiprocessing as mp


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def pack_q1(res):
    """oracle.q1 dict -> vd_partials bytes of plans.q1() (6 groups x 7 slots)."""
    b = bytearray(6 * 7 * 16)
    for g in range(6):
        vals = res.get(g, [0] * 6)
        rows = vals[5] if g in res else 0
        for a, v in enumerate(list(vals) + [rows]):
            struct.pack_into("<Qq", b, (g * 7 + a) * 16, v & (2**64 - 1), v >> 64)
    return bytes(b)


def _worker(rank, world, port, ret):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    import sys
    sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
    import torch
    import torch.distributed as dist

    import gen
    import oracle
    from paper_journals_pvldb_pirkmzm16_b200 import dist as vdist
    from paper_journals_pvldb_pirkmzm16_b200 import plans

    dist.init_process_group("gloo", rank=rank, world_size=world)
    sf = 0.002
    n = gen.lineitem_rows(sf)
    a, b = vdist.shard_range(n, rank, world, align=16)
    li = {k: gen.host(c, b - a, a, sf=sf) for k, c in gen.LINEITEM_COLS.items()}
    local = torch.frombuffer(bytearray(pack_q1(oracle.q1(li))), dtype=torch.uint8)
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    plan = plans.q1()
    # the merge reads only the columns' dtypes (int128 vs f64 addition)
    views = [vd.column_meta(gen.dtype_of(gen.LINEITEM_COLS[c])) for c in plans.Q1_COLS]
    merged = vdist.exchange_and_merge(plan, views, [], local)
    ret[rank] = {k: v[:6] for k, v in merged.items()}
    dist.destroy_process_group()


def test_shard_range_covers_rows_exactly():
    from paper_journals_pvldb_pirkmzm16_b200.dist import shard_range
    for n in [0, 1, 17, 600037]:
        for G in [1, 2, 3, 8]:
            for al in [1, 16]:
                rs = [shard_range(n, r, G, al) for r in range(G)]
                assert rs[0][0] == 0 and rs[-1][1] == n
                assert all(rs[i][1] == rs[i + 1][0] for i in range(G - 1))
                assert all(x[0] % al == 0 for x in rs)


@pytest.mark.parametrize("world", [2])
def test_gloo_exchange_and_merge_equals_whole(world):
    import gen
    import oracle
    ctx = mp.get_context("spawn")
    mgr = ctx.Manager()
    ret = mgr.dict()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, ret)) for r in range(world)]
    for p in procs:
        p.start()
    for p in procs:
        p.join(180)
        assert p.exitcode == 0
    sf = 0.002
    n = gen.lineitem_rows(sf)
    whole = oracle.q1({k: gen.host(c, n, sf=sf) for k, c in gen.LINEITEM_COLS.items()})
    for r in range(world):
        assert dict(ret[r]) == whole
