"""GPU parity of the single operators through the C ABI vs the CPU oracle.

Selection positions, gathers, scatters, partitions and integer folds must be
bit-exact; float folds agree within 1e-9 relative (BASELINE.json north_star)
-- the oracle accumulates in long double, the GPU in f64.
"""
import zlib

import numpy as np
import pytest
import torch

import gen
import oracle
from paper_journals_pvldb_pirkmzm16_b200 import vd
from vd_testutil import cuda_tensor, i128_from_bytes, minmax, with_eps

pytestmark = pytest.mark.gpu

SIZES = [0, 1, 3, 15, 16, 17, 127, 128, 129, 4095, 4096, 4097, 3 * 4096 + 5, 65536 + 7]
REL = 1e-9


# ---------------------------------------------------------------------------
# oracle helpers
# ---------------------------------------------------------------------------
def oracle_runs(ctrl_vals):
    """Run starts of a control vector per the oracle (FoldCount is non-epsilon
    exactly at run starts)."""
    p = oracle.run("c := FoldCount(k, k)", k=np.asarray(ctrl_vals, dtype=np.int64))
    return [i for i, x in enumerate(p.get("c")) if x is not None]


def ctrl_values(kind, n, seed=0):
    """Materialised values of the control vector of `kind` (for the oracle)."""
    i = np.arange(n, dtype=np.int64)
    if kind is None:
        return np.zeros(n, dtype=np.int64), None
    if kind[0] == "fixed":
        R = kind[1]
        return i // R, vd.ctrl(0, 1, R)
    if kind[0] == "virtual":
        num, den, cap = kind[1], kind[2], kind[3]
        v = (i * num) // den
        if cap:
            v = v % cap
        return v, vd.ctrl(0, num, den, cap)
    if kind[0] == "mat":
        rng = np.random.default_rng(seed)
        lens = []
        tot = 0
        while tot < n:
            L = int(rng.choice([1, 1, 2, 3, 5, 17, 100, 4096, 5000]))
            lens.append(L)
            tot += L
        vals = np.repeat(rng.integers(0, 3, size=len(lens)), lens)[:n].astype(np.int64)
        return vals, "mat"
    raise ValueError(kind)


def make_ctrl(kind, n, seed=0):
    vals, c = ctrl_values(kind, n, seed)
    keep = None
    if c == "mat":
        keep = cuda_tensor(vals.astype(np.int32))
        c = vd.ctrl(materialized=keep)
    return vals, c, keep


CTRLS = [None, ("fixed", 4), ("fixed", 1000), ("fixed", 4096), ("virtual", 2, 3, 0), ("virtual", 3, 1, 3),
         ("mat",)]


# ---------------------------------------------------------------------------
# a2+a3 selection
# ---------------------------------------------------------------------------
@pytest.mark.parametrize("mode", ["branch", "predicated"])
@pytest.mark.parametrize("n", SIZES + [1 << 20, (1 << 20) + 3])
def test_select_f32_single_term_vs_oracle(mode, n):
    v = gen.host(gen.F32_UNIFORM, n, seed=11)
    t = float(np.float32(0.5))
    pos_o, cnt_o, _ = oracle.select_f32(v, t, "lt")
    dv = cuda_tensor(v)
    out = torch.empty(max(n, 1), dtype=torch.int32, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    fn([vd.column(dv)], n, vd.pred([[(0, "<", t)]]), out_pos=out, out_count=cnt)
    c = int(cnt.item())
    assert c == cnt_o
    assert np.array_equal(out[:c].cpu().numpy(), pos_o)


@pytest.mark.parametrize("mode", ["branch", "predicated"])
@pytest.mark.parametrize("shift", [1, 2, 3])
def test_select_into_unaligned_output_vs_oracle(mode, shift):
    """Positions written to an out_pos that starts 4, 8 or 12 bytes past a
    16-byte boundary (the position pass's vector flush aligns on the output
    address), selectivities from sparse to dense, ragged n."""
    n = 300007
    v = gen.host(gen.F32_UNIFORM, n, seed=29)
    dv = cuda_tensor(v)
    for t in (0.01, 0.5, 0.97):
        t = float(np.float32(t))
        pos_o, cnt_o, _ = oracle.select_f32(v, t, "lt")
        buf = torch.full((n + 8,), -7, dtype=torch.int32, device="cuda")
        out = buf[shift:shift + n]
        cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
        fn = vd.select_branch if mode == "branch" else vd.select_predicated
        fn([vd.column(dv)], n, vd.pred([[(0, "<", t)]]), out_pos=out, out_count=cnt)
        c = int(cnt.item())
        assert c == cnt_o
        assert np.array_equal(out[:c].cpu().numpy(), pos_o)
        assert (buf[:shift] == -7).all().item()  # nothing written before out_pos


@pytest.mark.parametrize("mode", ["branch", "predicated"])
@pytest.mark.parametrize("dtype", ["u8", "i32", "i64", "f64"])
@pytest.mark.parametrize("n", [0, 5, 4097, 70001])
def test_select_dtypes_with_eps_vs_interpreter(mode, dtype, n):
    rng = np.random.default_rng(n + 3)
    if dtype == "u8":
        a = rng.integers(0, 200, n).astype(np.uint8)
        op, c = ">", 100
    elif dtype == "i32":
        a = rng.integers(-1000, 1000, n).astype(np.int32)
        op, c = "<=", 17
    elif dtype == "i64":
        a = rng.integers(-10**15, 10**15, n).astype(np.int64)
        op, c = "!=", int(a[0]) if n else 0
    else:
        a = rng.random(n) * 10
        op, c = ">=", 3.5
    a, m = with_eps(a, 0.05, n)
    # oracle: epsilon slots are not selected (reading A9)
    prog = {">": "p := Greater(v, %s)", "<=": "p := Greater(%s, v)", "!=": "e := Equals(v, %s)",
            ">=": "p := Greater(v, %s)"}[op]
    cc = c
    if op == "<=":
        cc = c + 1
    if op == ">=":
        cc = np.nextafter(c, -np.inf)  # x >= c == x > pred(c) for doubles
    prog = prog % (float(cc).hex() if dtype == "f64" else repr(cc))
    if op == "!=":
        prog += "\np := Equals(e, 0)"
    prog += "\npos := FoldSelect(p)"
    vals = a.astype(np.float64) if dtype == "f64" else a.astype(np.int64)
    p = oracle.run(prog, v=(vals, m))
    exp = [x for x in p.get("pos") if x is not None]
    dv = cuda_tensor(a)
    out = torch.empty(max(n, 1), dtype=torch.int32, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    fn([vd.column(dv)], n, vd.pred([[(0, op, c)]]), out_pos=out, out_count=cnt)
    k = int(cnt.item())
    assert out[:k].cpu().tolist() == exp


@pytest.mark.parametrize("mode", ["branch", "predicated"])
def test_select_generic_multi_column_or_of_ands(mode):
    """A disjunction of conjunctions over three columns (generic flag path)."""
    n = 50000
    rng = np.random.default_rng(5)
    a = rng.integers(0, 100, n).astype(np.int32)
    b = rng.integers(0, 7, n).astype(np.uint8)
    c = rng.random(n).astype(np.float32)
    p = vd.pred([[(0, ">", 50), (1, "in", [1, 3])], [(2, "<", 0.1)], [(0, "==", 7), (2, ">=", 0.5)]])
    exp = np.flatnonzero(((a > 50) & np.isin(b, [1, 3])) | (c < np.float32(0.1)) | ((a == 7) & (c >= 0.5)))
    # same predicate through the oracle interpreter
    prog = """
    g1 := Greater(a, 50)
    e1 := Equals(b, 1)
    e3 := Equals(b, 3)
    in1 := LogicalOr(e1, e3)
    c1 := LogicalAnd(g1, in1)
    c2 := Greater(%s, c)
    e7 := Equals(a, 7)
    g5 := Greater(c, %s)
    c3 := LogicalAnd(e7, g5)
    o1 := LogicalOr(c1, c2)
    p := LogicalOr(o1, c3)
    pos := FoldSelect(p)
    """ % (float(np.float32(0.1)).hex(), float(np.nextafter(0.5, 0)).hex())
    po = oracle.run(prog, a=a, b=b, c=c.astype(np.float64))
    got_o = [x for x in po.get("pos") if x is not None]
    assert got_o == exp.tolist()
    out = torch.empty(n, dtype=torch.int32, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    fn([vd.column(cuda_tensor(a)), vd.column(cuda_tensor(b)), vd.column(cuda_tensor(c))], n, p, out_pos=out,
       out_count=cnt)
    k = int(cnt.item())
    assert out[:k].cpu().tolist() == got_o


@pytest.mark.parametrize("kind", CTRLS)
@pytest.mark.parametrize("n", [1, 4097, 30011])
def test_fold_select_run_alignment_vs_interpreter(kind, n):
    """FoldSelect(.fold, .s) (Fig 9): positions per run, suppressed
    form = ascending list + run offsets (reading A4)."""
    rng = np.random.default_rng(n)
    s = (rng.random(n) < 0.3).astype(np.int32)
    cvals, c, keep = make_ctrl(kind, n, seed=n)
    p = oracle.run("pos := FoldSelect(k, s)", k=cvals, s=s)
    padded = p.get("pos")
    starts = oracle_runs(cvals)
    bounds = starts + [n]
    exp_pos, exp_off = [], [0]
    for r in range(len(starts)):
        seg = [x for x in padded[bounds[r]:bounds[r + 1]] if x is not None]
        exp_pos += seg
        exp_off.append(exp_off[-1] + len(seg))
    out = torch.empty(n, dtype=torch.int32, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    off = torch.full((n + 2,), -7, dtype=torch.int64, device="cuda")
    nr = torch.zeros(1, dtype=torch.int64, device="cuda")
    for mode in [vd.VD_SEL_BRANCH, vd.VD_SEL_PREDICATED]:
        vd.fold_select(vd.column(cuda_tensor(s)), c, mode, out_pos=out, out_count=cnt, out_run_off=off,
                       out_nruns=nr)
        k = int(cnt.item())
        assert out[:k].cpu().tolist() == exp_pos
        R = int(nr.item())
        assert R == len(starts)
        assert off[:R + 1].cpu().tolist() == exp_off


# ---------------------------------------------------------------------------
# a6 folds
# ---------------------------------------------------------------------------
def _run_fold(op, a, c, n, dtype_np):
    dv = cuda_tensor(a)
    col = vd.column(dv, length=n)
    nr = torch.zeros(1, dtype=torch.int64, device="cuda")
    cap = max(n, 1)
    counts = torch.zeros(cap, dtype=torch.int64, device="cuda")
    if op == "sum":
        isf = dtype_np.kind == "f"
        out = torch.zeros(cap * (1 if isf else 2), dtype=torch.float64 if isf else torch.int64, device="cuda")
        vd.fold_sum(col, c, out=out, out_counts=counts, out_nruns=nr)
    elif op == "count":
        out = torch.zeros(cap, dtype=torch.int64, device="cuda")
        vd.fold_count(col, c, out=out, out_nruns=nr)
    else:
        out = torch.zeros(cap, dtype=dv.dtype, device="cuda")
        (vd.fold_min if op == "min" else vd.fold_max)(col, c, out=out, out_counts=counts, out_nruns=nr)
    R = int(nr.item())
    return out, counts, R


@pytest.mark.parametrize("op", ["sum", "count", "min", "max"])
@pytest.mark.parametrize("dtype", ["u8", "i32", "i64", "f32", "f64"])
@pytest.mark.parametrize("kind", CTRLS)
def test_fold_vs_interpreter(op, dtype, kind):
    n = 20011
    rng = np.random.default_rng(zlib.crc32(repr((op, dtype, kind)).encode()))
    if dtype == "u8":
        a = rng.integers(0, 250, n).astype(np.uint8)
    elif dtype == "i32":
        a = rng.integers(-2**31 + 1, 2**31 - 1, n).astype(np.int32)
    elif dtype == "i64":
        a = rng.integers(-2**62, 2**62, n).astype(np.int64)
    elif dtype == "f32":
        a = rng.random(n).astype(np.float32)
    else:
        a = rng.standard_normal(n) * 1e6
    a, m = with_eps(a, 0.1, 1)
    # an all-epsilon stretch (all-epsilon runs for short run lengths, reading A5)
    if dtype in ("u8", "i32", "i64"):
        a[100:140] = {"u8": 0xFF, "i32": -2**31, "i64": -2**63}[dtype]
    else:
        a[100:140] = np.nan
    m[100:140] = True
    cvals, c, keep = make_ctrl(kind, n, seed=7)
    vals = a.astype(np.float64) if a.dtype.kind == "f" else a.astype(np.int64)
    fname = {"sum": "FoldSum", "count": "FoldCount", "min": "FoldMin", "max": "FoldMax"}[op]
    p = oracle.run(f"r := {fname}(k, v)\ncn := FoldCount(k, v)", k=cvals, v=(vals, m))
    starts = oracle_runs(cvals)
    exp = [p.get("r")[s] for s in starts]
    exp_cnt = [p.get("cn")[s] for s in starts]
    out, counts, R = _run_fold(op, a, c, n, a.dtype)
    assert R == len(starts)
    o = out.cpu().numpy()
    if op == "sum" and a.dtype.kind != "f":
        got = [i128_from_bytes(o.tobytes(), r) for r in range(R)]
        assert got == exp
    elif op == "sum":
        ve, re_, _ = p.get_float_exact("r")
        for r, s in enumerate(starts):
            ref = ve[s] + re_[s]
            assert abs(o[r] - ref) <= REL * max(abs(ref), 1e-300) + 1e-300 * 0, (r, o[r], ref)
    elif op == "count":
        assert o[:R].tolist() == exp
    else:
        for r in range(R):
            if exp[r] is None:
                if a.dtype.kind == "f":
                    assert np.isnan(o[r])
                else:
                    assert int(o[r]) == {"u8": 0xFF, "i32": -2**31, "i64": -2**63}[dtype]
            else:
                assert float(o[r]) == float(exp[r]) if a.dtype.kind == "f" else int(o[r]) == exp[r]
    if op != "count":
        assert counts[:R].cpu().tolist() == exp_cnt


@pytest.mark.parametrize("n", [0, 1, 4096, 4097, 1 << 20])
def test_fold_sum_one_run_closed_form(n):
    """FoldSum of Range(0, n, 1) = n(n-1)/2 (closed form, exact in 128 bits)."""
    a = np.arange(n, dtype=np.int64)
    out, counts, R = _run_fold("sum", a, None, n, a.dtype)
    assert R == (1 if n else 0)
    if n:
        assert i128_from_bytes(out.cpu().numpy().tobytes(), 0) == n * (n - 1) // 2


def test_hierarchical_fold_fig3_fig4_on_gpu():
    """Fig 3/4: FoldSum over runs of 1024, then FoldSum of the
    partials, equals the one-run FoldSum."""
    n = 300007
    a = gen.host(gen.I64_UNIFORM, n, p0=-10**12, p1=10**12)
    o1, _, R1 = _run_fold("sum", a, vd.ctrl(0, 1, 1024), n, a.dtype)
    part = np.array([i128_from_bytes(o1.cpu().numpy().tobytes(), r) for r in range(R1)], dtype=np.int64)
    o2, _, _ = _run_fold("sum", part, None, R1, part.dtype)
    o3, _, _ = _run_fold("sum", a, None, n, a.dtype)
    tot = i128_from_bytes(o2.cpu().numpy().tobytes(), 0)
    assert tot == i128_from_bytes(o3.cpu().numpy().tobytes(), 0) == int(a.astype(object).sum())


@pytest.mark.parametrize("dtype", ["u8", "i32", "i64", "f32", "f64"])
@pytest.mark.parametrize("kind", CTRLS)
@pytest.mark.parametrize("n", [0, 1, 4095, 4096, 70001])
def test_fold_scan_vs_interpreter(dtype, kind, n):
    """FoldScan (Table 2; reading A27): per-run inclusive prefix sums
    restarting at each run, epsilon slots stay epsilon, against the oracle's
    FoldScan -- across tile boundaries (4096-row tiles), runs shorter and
    longer than a tile, irregular virtual and materialized controls.  Integer
    exact; float within 1e-9 relative of the long-double oracle (positive
    data: no cancellation)."""
    rng = np.random.default_rng(zlib.crc32(repr((dtype, kind, n)).encode()))
    if dtype == "u8":
        a = rng.integers(0, 250, n).astype(np.uint8)
    elif dtype == "i32":
        a = rng.integers(-2**31 + 1, 2**31 - 1, n).astype(np.int32)
    elif dtype == "i64":
        a = rng.integers(-2**40, 2**40, n).astype(np.int64)
    elif dtype == "f32":
        a = rng.random(n).astype(np.float32)
    else:
        a = rng.random(n) * 1e6
    a, m = with_eps(a, 0.05, 3)
    cvals, c, keep = make_ctrl(kind, n, seed=9)
    dv = cuda_tensor(a)
    col = vd.column(dv, minmax=(-2**40, 2**40) if dtype == "i64" else None)
    isf = a.dtype.kind == "f"
    out = torch.full((max(n, 1),), 7, dtype=torch.float64 if isf else torch.int64, device="cuda")
    vd.fold_scan(col, c, out=out)
    assert vd.last_launch_count() == (1 if n else 0)
    if n == 0:
        return
    vals = a.astype(np.float64) if isf else a.astype(np.int64)
    p = oracle.run("r := FoldScan(k, v)", k=cvals, v=(vals, m))
    o = out[:n].cpu().numpy()
    if isf:
        ve, re_, e = p.get_float_exact("r")
        assert np.array_equal(np.isnan(o), e)
        ref = ve[~e] + re_[~e]
        assert np.all(np.abs(o[~e] - ref) <= REL * np.abs(ref) + 1e-300)
    else:
        ev, ee = p.get_arrays("r")
        assert np.array_equal(o == -2**63, ee)
        assert np.array_equal(o[~ee], np.asarray(ev)[~ee].astype(np.int64))


# ---------------------------------------------------------------------------
# a4 gather, a5 scatter / partition
# ---------------------------------------------------------------------------
@pytest.mark.parametrize("n", [0, 1, 1023, 100003])
@pytest.mark.parametrize("bias", [0, 1])
def test_gather_multi_vs_interpreter(n, bias):
    rng = np.random.default_rng(n + bias)
    m = 5000
    srcs = [rng.integers(0, 255, m).astype(np.uint8), rng.integers(-10**6, 10**6, m).astype(np.int32),
            rng.integers(-10**15, 10**15, m).astype(np.int64), rng.random(m).astype(np.float32)]
    pos = rng.integers(-3, m + 4, n).astype(np.int32)  # includes OOB and negative (epsilon)
    dpos = cuda_tensor(pos)
    outs = [torch.empty(max(n, 1), dtype=cuda_tensor(s[:1]).dtype, device="cuda") for s in srcs]
    vd.gather_multi([vd.column(cuda_tensor(s)) for s in srcs], dpos, n, bias, outs)
    p_ = pos.astype(np.int64) - bias
    p_[pos < 0] = -1  # a negative position is epsilon before the bias applies
    for s, o in zip(srcs, outs):
        po = oracle.run("g := Gather(s, p)", s=s.astype(np.float64 if s.dtype.kind == "f" else np.int64), p=p_)
        vals, eps = po.get_arrays("g")
        got = o[:n].cpu().numpy()
        if s.dtype.kind == "f":
            assert np.array_equal(np.isnan(got), eps)
            assert np.array_equal(got[~eps].astype(np.float64), vals[~eps])
        else:
            sentinel = {"uint8": 0xFF, "int32": -2**31, "int64": -2**63}[s.dtype.name]
            exp = np.where(eps, sentinel, vals).astype(np.int64)
            assert np.array_equal(got.astype(np.int64), exp)


@pytest.mark.parametrize("fields", [("i32", "i32"), ("u8", "i64", "i32"), ("f32", "i64", "u8", "i32"),
                                    ("i64", "i64", "i64", "i64"), ("f64",)])
@pytest.mark.parametrize("n", [0, 1, 4097, 200003])
def test_layout_transform_vs_interpreter(fields, n):
    """Fig 14 Layout Transform: vd_zip materialises the target
    columns row-wise, vd_gather_rows resolves positions into the rows; every
    field equals the oracle's Gather(Zip(...), p) (epsilon in the columns,
    negative and out-of-bounds positions give epsilon, reading A11)."""
    rng = np.random.default_rng(n + len(fields))
    m = 3001
    gen_ = {"u8": lambda: rng.integers(0, 255, m).astype(np.uint8),
            "i32": lambda: rng.integers(-10**9, 10**9, m).astype(np.int32),
            "i64": lambda: rng.integers(-10**17, 10**17, m).astype(np.int64),
            "f32": lambda: rng.random(m).astype(np.float32),
            "f64": lambda: rng.random(m)}
    cols = [gen_[f]() for f in fields]
    eps = [rng.random(m) < 0.02 for _ in fields]
    for c, e in zip(cols, eps):
        c[e] = {"u1": 0xFF, "i4": -2**31, "i8": -2**63, "f4": np.nan, "f8": np.nan}[c.dtype.kind + str(c.itemsize)]
    pos = rng.integers(-2, m + 3, n).astype(np.int32)
    dts = [{"u8": vd.VD_U8, "i32": vd.VD_I32, "i64": vd.VD_I64, "f32": vd.VD_F32, "f64": vd.VD_F64}[f] for f in fields]
    offs, stride = vd.row_layout(dts)
    dcols = [cuda_tensor(c) for c in cols]
    rows = torch.empty(m * stride, dtype=torch.uint8, device="cuda")
    vd.zip_rows([vd.column(c) for c in dcols], rows)
    outs = [torch.empty(max(n, 1), dtype=d.dtype, device="cuda") for d in dcols]
    vd.gather_rows(rows, m, dts, cuda_tensor(pos), n, 1, outs)
    assert vd.last_launch_count() == (1 if n else 0)
    # row bytes: each field at its offset, padding zero
    rb = rows.cpu().numpy().reshape(m, stride)
    for c, o in zip(cols, offs):
        assert np.array_equal(rb[:, o:o + c.itemsize].copy().view(c.dtype).reshape(-1).view(np.uint8),
                              c.view(np.uint8))
    p_ = pos.astype(np.int64) - 1
    p_[pos < 0] = -1
    names = [f"f{k}" for k in range(len(fields))]
    # Zip needs two or more inputs (Table 2); one field is a plain Gather
    prog = (f"z := Zip({', '.join('t.' + x for x in names)})\ng := Gather(z, p)" if len(names) > 1
            else "g := Gather(t.f0, p)")
    po = oracle.run(prog, p=p_, **{f"t__{x}": (c.astype(np.float64 if c.dtype.kind == "f" else np.int64), e)
                                    for x, c, e in zip(names, cols, eps)})
    for x, c, o in zip(names, cols, outs):
        vals, e = po.get_arrays(f"g.{x}" if len(names) > 1 else "g")
        got = o[:n].cpu().numpy()
        if c.dtype.kind == "f":
            assert np.array_equal(np.isnan(got), e)
            assert np.array_equal(got[~e].astype(np.float64), vals[~e])
        else:
            sentinel = {"uint8": 0xFF, "int32": -2**31, "int64": -2**63}[c.dtype.name]
            assert np.array_equal(got.astype(np.int64), np.where(e, sentinel, vals).astype(np.int64))


@pytest.mark.parametrize("n,out_len", [(0, 5), (1, 1), (5000, 100), (100000, 70000), (3, 0)])
def test_scatter_last_writer_wins_vs_interpreter(n, out_len):
    rng = np.random.default_rng(n)
    v = rng.integers(-10**12, 10**12, n).astype(np.int64)
    pos = rng.integers(-2, out_len + 3, n).astype(np.int32)
    out = torch.empty(max(out_len, 1), dtype=torch.int64, device="cuda")
    vd.scatter(vd.column(cuda_tensor(v)), cuda_tensor(pos), n, out, out_len)
    po = oracle.run("o := Scatter(v, %d, p)" % out_len, v=v, p=pos.astype(np.int64))
    exp = po.get("o")
    got = out[:out_len].cpu().tolist()
    assert got == [(-2**63 if e is None else e) for e in exp]


def test_scatter_permutation_unique():
    n = 123457
    pi = gen.host(gen.I32_PERM, n, p0=n, seed=3)
    v = gen.host(gen.F32_UNIFORM, n, seed=4)
    out = torch.empty(n, dtype=torch.float32, device="cuda")
    vd.scatter(vd.column(cuda_tensor(v)), cuda_tensor(pi), n, out, n, unique=True)
    po = oracle.run("o := Scatter(v, %d, p)" % n, v=v.astype(np.float64), p=pi.astype(np.int64))
    exp = np.array(po.get("o"), dtype=np.float64)  # a permutation: every slot written (no epsilon)
    assert np.array_equal(out.cpu().numpy().astype(np.float64), exp)


@pytest.mark.parametrize("n,P", [(0, 4), (10, 4), (4097, 6), (300001, 175), (70000, 1024)])
def test_partition_vs_interpreter(n, P):
    """Partition(V1.v, Range(from, P, 1)) (reading A13, Fig 11)."""
    rng = np.random.default_rng(P)
    frm = 3
    v = rng.integers(frm - 2, frm + P + 2, n).astype(np.int32)  # some below / above the pivots
    v, m = with_eps(v, 0.02, 9)
    out = torch.empty(max(n, 1), dtype=torch.int32, device="cuda")
    bc = torch.zeros(P, dtype=torch.int64, device="cuda")
    vd.partition(vd.column(cuda_tensor(v)), frm, P, out, bc)
    po = oracle.run("piv := Range(%d, %d, 1)\npos := Partition(v, piv)" % (frm, P), v=(v.astype(np.int64), m))
    exp = po.get("pos")
    assert out[:n].cpu().tolist() == [(-1 if e is None else e) for e in exp]
    b = np.clip(v[~m].astype(np.int64) - frm, 0, P - 1)
    assert bc.cpu().tolist() == np.bincount(b, minlength=P).tolist()


@pytest.mark.gpu
@pytest.mark.parametrize("mode", ["branch", "predicated"])
@pytest.mark.parametrize("dtype", ["u8", "i32", "f32"])
@pytest.mark.parametrize("offset", [0, 4])
def test_select_flag_pass_tiles_and_tail(mode, dtype, offset):
    """Several 16384-row tiles of the TMA flag pass plus a ragged LDG tail; a
    base pointer 4 bytes past a 16-byte boundary takes the LDG pass instead.
    Positions must equal the interpreter's FoldSelect of the predicate
    (P:L101-108)."""
    n = 5 * 16384 + 1000 + 7
    rng = np.random.default_rng(99)
    if dtype == "u8":
        a = rng.integers(0, 255, n + 16).astype(np.uint8)  # 0xFF = epsilon excluded by the interval
        op, c = ">", 100
        prog = "p := Greater(v, 100)"
    elif dtype == "i32":
        a = rng.integers(-1000, 1000, n + 16).astype(np.int32)
        op, c = "<=", 17
        prog = "p := Greater(18, v)"
    else:
        a = rng.random(n + 16).astype(np.float32)
        op, c = "<", 0.25
        prog = "p := Greater(%s, v)" % float(np.float32(0.25)).hex()
    eps = (a == 0xFF) if dtype == "u8" else np.zeros(a.size, bool)
    esz = a.itemsize
    skip = offset // esz
    da = cuda_tensor(a)[skip:skip + n]
    w = a[skip:skip + n]
    vals = w.astype(np.float64) if dtype == "f32" else w.astype(np.int64)
    po = oracle.run(prog + "\npos := FoldSelect(p)", v=(vals, eps[skip:skip + n]))
    exp = np.array([x for x in po.get("pos") if x is not None], dtype=np.int64)
    out = torch.empty(n, dtype=torch.int32, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    fn([vd.column(da)], n, vd.pred([[(0, op, c)]]), out_pos=out, out_count=cnt)
    k = int(cnt.item())
    assert k == len(exp)
    assert np.array_equal(out[:k].cpu().numpy(), exp)
