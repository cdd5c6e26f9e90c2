"""CPU checks of the C-ABI boundary: libvd.so loads, exports every function
include/vd.h declares, its structs match the binding, and the host-only
logic (control-vector run counting, workspace sizing, argument validation,
the cross-device merge) behaves.  No kernel is launched here."""
import ctypes
import os
import re
import struct

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def declared_functions():
    src = open(os.path.join(ROOT, "include", "vd.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    names = set(re.findall(r"^\s*(?:const\s+)?(?:vd_status|size_t|int32_t|const char\*|void)\s*\*?\s*(vd_\w+)\s*\(",
                           src, flags=re.M))
    return sorted(names)


def test_header_declares_the_north_star_calls():
    names = declared_functions()
    for want in ["vd_load_column", "vd_select_branch", "vd_select_predicated", "vd_gather", "vd_scatter",
                 "vd_fold_sum", "vd_fold_count", "vd_fold_min", "vd_fold_max", "vd_fold_select", "vd_run_pipeline",
                 "vd_merge_partials", "vd_merge_partials_device", "vd_workspace_bytes", "vd_partition",
                 "vd_hash_group_fold", "vd_merge_groups"]:
        assert want in names


def test_library_exports_every_declared_symbol():
    lib = ctypes.CDLL(os.path.join(ROOT, "paper_journals_pvldb_pirkmzm16_b200", "libvd.so"))
    missing = [n for n in declared_functions() if not hasattr(lib, n)]
    assert missing == []
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    assert set(declared_functions()) == set(vd.EXPORTS)


def test_struct_layout_matches_binding():
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    vd._check_abi()
    assert ctypes.sizeof(vd.vd_column) == 48
    assert vd.version().startswith("voodoo-b200")


def test_ctrl_run_counts_reading_A2():
    """Run metadata: Divide(Range, R) -> runs of R; Modulo with
    cap 1 or step 0 -> one run; integer step k -> runs of 1 unless cap | k."""
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    assert vd.ctrl_runs(None, 10) == 1
    assert vd.ctrl_runs(None, 0) == 0
    assert vd.ctrl_runs(vd.ctrl(0, 1, 4), 10) == 3
    assert vd.ctrl_runs(vd.ctrl(0, 1, 4, cap=2), 10) == 3
    assert vd.ctrl_runs(vd.ctrl(0, 0, 1), 10) == 1
    assert vd.ctrl_runs(vd.ctrl(0, 1, 1, cap=1), 10) == 1
    assert vd.ctrl_runs(vd.ctrl(0, 2, 1, cap=2), 10) == 1
    assert vd.ctrl_runs(vd.ctrl(0, 2, 1, cap=3), 10) == 10
    assert vd.ctrl_runs(vd.ctrl(0, 1, 100), 10) == 1
    with pytest.raises(vd.VdError):
        vd.ctrl_runs(vd.ctrl(0, 2, 3), 10)  # irregular runs: data dependent (device count)
    with pytest.raises(vd.VdError):
        vd.ctrl_runs(vd.ctrl(0, 1, 0), 10)  # den 0


def test_workspace_sizes_grow_and_validate():
    from paper_journals_pvldb_pirkmzm16_b200 import plans, vd
    a = vd.workspace_bytes(vd.VD_OP_SELECT, 1000)
    b = vd.workspace_bytes(vd.VD_OP_SELECT, 10**8)
    assert 0 < a < b
    assert vd.workspace_bytes(vd.VD_OP_FOLD, 10**6, vd.ctrl(0, 2, 3)) > vd.workspace_bytes(vd.VD_OP_FOLD, 10**6)
    assert vd.workspace_bytes(vd.VD_OP_PIPELINE, 10**6, None, plans.q1()) > 0
    assert vd.partials_bytes(plans.q1()) == 6 * 7 * 16


def test_validation_errors_are_synchronous():
    """Argument errors come back before any launch (include/vd.h 'Errors')."""
    from paper_journals_pvldb_pirkmzm16_b200 import plans, vd
    plan = plans.q1()
    c = vd.vd_column()
    c.dtype, c.len = vd.VD_I32, 10
    cols = (vd.vd_column * 7)(*([c] * 7))
    st = vd._L.vd_run_pipeline(ctypes.byref(plan), cols, 7, 10, None, 0, None, None, 0, None)
    assert st == vd.VD_E_NULL
    # key domain proof from metadata: rf in [0, 9] cannot fit 6 groups -> VD_E_DOMAIN
    cs = []
    for k, dt in enumerate([vd.VD_I32, vd.VD_U8, vd.VD_U8, vd.VD_I64, vd.VD_I64, vd.VD_I64, vd.VD_I64]):
        x = vd.vd_column()
        x.data, x.len, x.dtype = 4096, 10, dt
        if k in (1, 2):
            x.min, x.max, x.has_minmax = 0, 9, 1
        cs.append(x)
    arr = (vd.vd_column * 7)(*cs)
    st = vd._L.vd_run_pipeline(ctypes.byref(plan), arr, 7, 10, None, 0, ctypes.c_void_p(4096),
                               ctypes.c_void_p(4096), 1 << 30, None)
    assert st == vd.VD_E_DOMAIN
    bad = vd.pipeline(ngroups=0)
    assert vd._L.vd_run_pipeline(ctypes.byref(bad), arr, 7, 10, None, 0, ctypes.c_void_p(1), ctypes.c_void_p(1),
                                 1 << 30, None) == vd.VD_E_ARG


def test_no_cpu_fallback_without_device():
    """Compute entry points refuse to run without a CUDA device."""
    import torch
    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    c = vd.vd_column()
    c.data, c.len, c.dtype = 4096, 4, vd.VD_I64
    out = ctypes.c_void_p(8192)
    st = vd._L.vd_fold_sum(ctypes.byref(c), None, out, None, None, ctypes.c_void_p(4096), 1 << 20, None)
    assert st == vd.VD_E_CUDA
    assert "no CPU fallback" in vd._L.vd_last_error().decode()


def _pack(vals):
    b = b""
    for v in vals:
        if isinstance(v, float):
            b += struct.pack("<dq", v, 0)
        else:
            b += struct.pack("<Qq", v & (2**64 - 1), v >> 64)
    return b


def test_merge_partials_rank_order_int128_and_empty_groups():
    """Cross-GPU step of the hierarchical fold (Fig 3 one level up): 128-bit
    sums, min/max over non-empty ranks, empty groups stay empty."""
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    plan = vd.pipeline(key=[(0, 0, 0, 1)], ngroups=3,
                       aggs=[("sum", [1]), ("min", [1]), ("max", [1]), ("count",)])
    c0 = vd.vd_column()
    c0.dtype = vd.VD_U8
    c1 = vd.vd_column()
    c1.dtype = vd.VD_I64
    big = 2**63 - 1
    r0 = _pack([big, 5, 9, 2, 2] + [0, 0, 0, 0, 0] + [7, -3, -3, 1, 1])
    r1 = _pack([big, 1, 4, 3, 3] + [0, 0, 0, 0, 0] + [0, 0, 0, 0, 0])
    res = vd.merge_partials(plan, [c0, c1], [], [r0, r1])
    assert res == {0: [2 * big, 1, 9, 5, 5], 2: [7, -3, -3, 1, 1]}
    assert list(res) == [0, 2]  # ascending key, the empty group 1 dropped (Fig 11, A16)
    # the dtypes decide int128 vs f64 addition: several partials need the views
    with pytest.raises(vd.VdError):
        vd.merge_partials(plan, [], [], [r0, r1])


def test_merge_partials_float_sum_and_single_partial_compaction():
    """f64 SUM slots add as doubles; one partial is compacted verbatim
    (decode_partials = vd_merge_partials with nparts = 1)."""
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    plan = vd.pipeline(key=[(0, 0, 0, 1)], ngroups=4, aggs=[("sum", [1]), ("count",)])
    c0 = vd.vd_column()
    c0.dtype = vd.VD_U8
    c1 = vd.vd_column()
    c1.dtype = vd.VD_F64
    r0 = _pack([0.25, 1, 1] + [0, 0, 0] + [0, 0, 0] + [1.5, 2, 2])
    r1 = _pack([0, 0, 0] + [0, 0, 0] + [2.0, 3, 3] + [0.125, 1, 1])
    assert vd.merge_partials(plan, [c0, c1], [], [r0, r1], float_aggs=[True]) == \
        {0: [0.25, 1, 1], 2: [2.0, 3, 3], 3: [1.625, 3, 3]}
    assert vd.decode_partials(r1, plan, float_aggs=[True]) == {2: [2.0, 3, 3], 3: [0.125, 1, 1]}


def test_binding_decodes_without_filtering():
    """The binding only decodes what the library's vd_result holds: a
    vd_result whose groups are written out of order and include a zero-row
    entry comes back exactly as written (no filtering, no sorting)."""
    import struct
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    plan = vd.pipeline(key=[(0, 0, 0, 1)], ngroups=4, aggs=[("count",)])
    keys = struct.pack("<qqq", 3, 0, 2)
    aggs = _pack([5, 0, 9])
    rows = struct.pack("<qqq", 5, 0, 9)
    assert list(vd.decode_result(keys, aggs, rows, 3, plan).items()) == [(3, [5, 5]), (0, [0, 0]), (2, [9, 9])]


def test_pipeline_descriptor_round_trip():
    from paper_journals_pvldb_pirkmzm16_b200 import plans, vd
    p = plans.q1()
    assert p.naggs == 6 and p.ngroups == 6 and p.nkeyparts == 2
    assert p.pred.conj[0].terms[0].cmp == vd.VD_CMP_LE and p.pred.conj[0].terms[0].ival == 10471
    q = vd.pred([[(0, "in", [0, 3, 63])]])
    assert q.conj[0].terms[0].ival == (1 | 8 | (1 << 63)) - (1 << 64)


def test_row_layout_reading_fig14():
    """vd_row_layout (host only): fields in order, each aligned to its size,
    no overlap, stride a power of two >= 8 holding the packed row, rows of
    more than 32 bytes refused (one sector per lookup)."""
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    size = {vd.VD_U8: 1, vd.VD_I32: 4, vd.VD_F32: 4, vd.VD_I64: 8, vd.VD_F64: 8}
    import itertools
    for k in range(1, 5):
        for dts in itertools.product(list(size), repeat=k):
            if sum(size[d] for d in dts) > 24:
                continue
            offs, stride = vd.row_layout(list(dts))
            assert stride >= 8 and stride & (stride - 1) == 0 and stride <= 32
            end = 0
            for d, o in zip(dts, offs):
                assert o % size[d] == 0 and o >= end
                end = o + size[d]
            assert end <= stride and stride // 2 < max(end, 5)
    assert vd.row_layout([vd.VD_I32, vd.VD_I32]) == ([0, 4], 8)
    with pytest.raises(vd.VdError):
        vd.row_layout([vd.VD_U8, vd.VD_F64, vd.VD_F64, vd.VD_F64, vd.VD_U8])


def test_group_fold_host_validation():
    """vd_group_fold (NEXT-4) validates before touching the device: the key's
    min/max metadata sizes the table (VD_E_DOMAIN without, or beyond
    VD_MAX_DOMAIN), integer SUMs must be provably exact (VD_E_OVERFLOW), the
    workspace is checked (VD_E_WORKSPACE), and without a GPU the call fails
    loudly (VD_E_CUDA: no CPU fallback)."""
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    L = vd._L

    def col(dt, lo=None, hi=None):
        c = vd.vd_column()
        c.data, c.len, c.dtype = 256, 1000, dt
        if lo is not None:
            c.min, c.max, c.has_minmax = lo, hi, 1
        return c

    out = ctypes.c_void_p(4096)

    def call(cols, aggs, ws=None, wsb=0):
        arr = (vd.vd_column * len(cols))(*cols)
        ag = vd.aggs_array(aggs)
        return L.vd_group_fold(arr, len(cols), 1000, None, 0, ag, len(aggs), out, out, out, out, ws, wsb, None)

    assert call([col(vd.VD_I64), col(vd.VD_I64, 0, 10)], [("count",)]) == vd.VD_E_DOMAIN
    assert call([col(vd.VD_I64, 0, 2**40), col(vd.VD_I64, 0, 10)], [("count",)]) == vd.VD_E_DOMAIN
    assert call([col(vd.VD_I64, 0, 99), col(vd.VD_I64, 0, 2**60)], [("sum", [1])]) == vd.VD_E_OVERFLOW
    assert call([col(vd.VD_I64, 0, 99), col(vd.VD_I64)], [("sum", [1])]) == vd.VD_E_OVERFLOW
    assert call([col(vd.VD_I64, 0, 99), col(vd.VD_F64)], [("min", [1])]) == vd.VD_E_UNSUPPORTED
    assert call([col(vd.VD_I64, 0, 99), col(vd.VD_I64, 0, 10)], [("sum", [1]), ("count",)]) == vd.VD_E_WORKSPACE
    need = vd.group_fold_ws_bytes(100, 2)
    assert need >= 100 * 3 * 8
    st = call([col(vd.VD_I64, 0, 99), col(vd.VD_I64, 0, 10)], [("sum", [1]), ("count",)], ctypes.c_void_p(1 << 20),
              need)
    assert st == vd.VD_E_CUDA


def test_fold_scan_host_validation():
    """vd_fold_scan: an i64 column needs min/max metadata proving its running
    sums fit int64 (VD_E_OVERFLOW otherwise); workspace checked; no GPU ->
    VD_E_CUDA."""
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    L = vd._L
    c = vd.vd_column()
    c.data, c.len, c.dtype = 256, 1000, vd.VD_I64
    out = ctypes.c_void_p(4096)
    assert L.vd_fold_scan(ctypes.byref(c), None, out, None, 0, None) == vd.VD_E_OVERFLOW
    c.min, c.max, c.has_minmax = -2**60, 2**60, 1
    assert L.vd_fold_scan(ctypes.byref(c), None, out, None, 0, None) == vd.VD_E_OVERFLOW
    c.min, c.max = -2**40, 2**40
    assert L.vd_fold_scan(ctypes.byref(c), None, out, None, 0, None) == vd.VD_E_WORKSPACE
    need = vd.workspace_bytes(vd.VD_OP_FOLD_SCAN, 1000)
    assert L.vd_fold_scan(ctypes.byref(c), None, out, ctypes.c_void_p(1 << 20), need, None) == vd.VD_E_CUDA


def test_workspace_grows_with_materialising_plans():
    """vd_workspace_bytes(VD_OP_PIPELINE): a Break plan needs n more bytes (one
    flag per row), a Materialize plan 4 B per row + 4 B per chunk more; a bad
    materialize value is refused (host only, no device needed)."""
    from paper_journals_pvldb_pirkmzm16_b200 import plans, vd
    n = 1_000_003
    base = vd.workspace_bytes(vd.VD_OP_PIPELINE, n, None, plans.q6())
    brk = plans.q6()
    brk.materialize = vd.VD_MAT_BREAK
    chk = plans.q6()
    chk.materialize, chk.mat_chunk = vd.VD_MAT_CHUNKS, 4096
    assert vd.workspace_bytes(vd.VD_OP_PIPELINE, n, None, brk) >= base + n
    nch = -(-n // 4096)
    assert vd.workspace_bytes(vd.VD_OP_PIPELINE, n, None, chk) >= base + 4 * nch * 4096 + 4 * nch
    bad = plans.q6()
    bad.materialize = 7
    with pytest.raises(vd.VdError):
        vd.workspace_bytes(vd.VD_OP_PIPELINE, n, None, bad)


def test_hash_and_merge_group_workspace_sizes():
    """The open-addressing tables are sized from the distinct-key bound
    (capacity: a power of two >= 2 x max_groups); the merge table holds
    16-byte aggregate slots."""
    from paper_journals_pvldb_pirkmzm16_b200 import vd
    a = vd.hash_group_fold_ws_bytes(1000, 2)
    b = vd.hash_group_fold_ws_bytes(100_000, 2)
    assert b > 50 * a // 2
    assert vd.merge_groups_ws_bytes(100_000, 2) > b  # 2 words per aggregate
    with pytest.raises(vd.VdError):
        vd.hash_group_fold_ws_bytes(0, 2)
