"""The single-launch selection kernels (k_sel_lag, the default at every size:
tiles counted into register-held words, counts published to a table, each
tile decoded LAG iterations later; k_sel_coop: per-CTA contiguous chunk
ranges streamed by TMA into ballot words, one grid barrier, in-order decode
into staged 16-byte stores) against the oracle: sizes from one row to
several 16-chunk tiles per CTA with a ragged end (TMA tiles, LDG for the
column's last partial chunk), all-false / all-true tiles, NaN (epsilon,
never selected: A9), int32 columns, unaligned outputs, branching and
predicated (identical positions), and the same inputs through
the 4-launch bitmap path (VD_SELECT_COOP=0) it replaces."""
import numpy as np
import pytest
import torch

import gen
import oracle
from paper_journals_pvldb_pirkmzm16_b200 import vd

from test_gpu_pipeline import env

pytestmark = pytest.mark.gpu

SIZES = [1, 31, 1023, 1024, 1025, 3 * 8192 + 5, 70001, 1 << 20, 148 * 16 * 1024 * 3 + 4097]


def _select(fn, v, n, t, shift=0):
    buf = torch.full((n + 8,), -7, dtype=torch.int32, device="cuda")
    out = buf[shift:shift + n]
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    fn([vd.column(v)], n, vd.pred([[(0, "<", t)]]), out_pos=out, out_count=cnt)
    c = int(cnt.item())
    assert (buf[:shift] == -7).all().item()
    assert (buf[shift + c:shift + c + 1] == -7).all().item() or c == n  # nothing past the count
    return out[:c].cpu().numpy()


@pytest.mark.parametrize("mode", ["branch", "predicated"])
@pytest.mark.parametrize("n", SIZES)
@pytest.mark.parametrize("t", [0.0, 0.001, 0.3, 1.0])
def test_fused_select_f32_vs_oracle(mode, n, t):
    v = gen.host(gen.F32_UNIFORM, n, seed=n % 977 + 5)
    v[::13] = np.nan  # epsilon
    t = float(np.float32(t))
    pos_o, cnt_o, _ = oracle.select_f32(v, t, "lt")
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    dv = torch.from_numpy(v).cuda()
    got = _select(fn, dv, n, t)
    assert len(got) == cnt_o and np.array_equal(got, pos_o)
    assert vd.last_fragment() == "sel_lag"
    with env(VD_SELECT_KERNEL="coop"):  # the single-barrier kernel agrees
        assert np.array_equal(_select(fn, dv, n, t), pos_o)
        assert vd.last_fragment() == "sel_coop"
    with env(VD_SELECT_COOP="0"):  # the bitmap path agrees
        assert np.array_equal(_select(fn, dv, n, t), pos_o)


@pytest.mark.parametrize("mode", ["branch", "predicated"])
@pytest.mark.parametrize("shift", [1, 2, 3])
def test_fused_select_unaligned_output(mode, shift):
    n = 5 * 8192 + 777
    v = gen.host(gen.F32_UNIFORM, n, seed=3)
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    dv = torch.from_numpy(v).cuda()
    for t in (0.02, 0.5, 0.99):
        t = float(np.float32(t))
        pos_o, _, _ = oracle.select_f32(v, t, "lt")
        assert np.array_equal(_select(fn, dv, n, t, shift), pos_o)


@pytest.mark.parametrize("mode", ["branch", "predicated"])
def test_fused_select_i32_tiles_alternating_empty_and_full(mode):
    """Tiles that select nothing next to tiles that select everything (the
    look-back sums zero and full aggregates), against the interpreter."""
    n = 9 * 8192 + 100
    rng = np.random.default_rng(1)
    a = rng.integers(-1000, 1000, n).astype(np.int32)
    tile = np.arange(n) // 8192
    a[tile % 3 == 0] = 5000   # never selected
    a[tile % 3 == 1] = -5000  # always selected
    a[::101] = -2**31         # epsilon: never selected (A9)
    m = a == -2**31
    p = oracle.run("p := Greater(17, v)\npos := FoldSelect(p)", v=(a.astype(np.int64), m))
    exp = np.array([x for x in p.get("pos") if x is not None])
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    da = torch.from_numpy(a).cuda()
    out = torch.empty(n, dtype=torch.int32, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    fn([vd.column(da)], n, vd.pred([[(0, "<", 17)]]), out_pos=out, out_count=cnt)
    k = int(cnt.item())
    assert np.array_equal(out[:k].cpu().numpy(), exp)


@pytest.mark.parametrize("mode", ["branch", "predicated"])
@pytest.mark.parametrize("n,t", [(10 * 10**6 + 3, 0.3), (50 * 10**6 + 17, 0.02), (50 * 10**6 + 17, 0.7),
                                 (120 * 10**6 + 1, 0.5), (37 * 10**6 + 4093, 0.002), (41 * 10**6 + 9, 0.12)])
def test_large_select_kernels_vs_oracle(mode, n, t):
    """The large-input kernels against the oracle's brute-force selection:
    the default lagged single pass (k_sel_lag: tile counts published to a
    table, each tile decoded LAG iterations later from register-held words;
    sparse / lane-owned / dense chunk paths) at both compiled lags, and the
    single-barrier kernel (k_sel_coop), at sizes with a ragged last tile,
    into an unaligned output."""
    v = gen.host(gen.F32_UNIFORM, n, seed=n % 1009)
    t = float(np.float32(t))
    pos_o, cnt_o, _ = oracle.select_f32(v, t, "lt")
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    dv = torch.from_numpy(v).cuda()
    got = _select(fn, dv, n, t, shift=1)
    assert vd.last_fragment() == "sel_lag"
    assert len(got) == cnt_o and np.array_equal(got, pos_o)
    with env(VD_SEL_LAG="16"):
        assert np.array_equal(_select(fn, dv, n, t), pos_o)
        assert vd.last_fragment() == "sel_lag"
    with env(VD_SELECT_KERNEL="coop"):
        assert np.array_equal(_select(fn, dv, n, t), pos_o)
        assert vd.last_fragment() == "sel_coop"


@pytest.mark.parametrize("mode", ["branch", "predicated"])
@pytest.mark.parametrize("mid", [None, "0", "640/1024", "640/100"])
def test_lag_select_chunk_density_mix(mode, mid):
    """Chunks of every density class of k_sel_lag's decode in one input
    (empty, <= SL_SPARSE, lane-owned, dense ballot blocks, full) with NaN
    epsilon rows, i32 and f32, against the oracle; the thresholds at their
    defaults, lane-owned off (every chunk through the ballot blocks), and
    lane-owned up to its maximum with the per-bit loop only / the fixed
    32-row loop above 100 positions."""
    n = 148 * 15 * 1024 * 6 + 12345
    rng = np.random.default_rng(7)
    chunk = np.arange(n) // 1024
    dens = np.array([0.0, 0.01, 0.04, 0.2, 0.31, 0.6, 1.0])[chunk % 7]
    v = np.where(rng.random(n) < dens, np.float32(0.25), np.float32(0.75)).astype(np.float32)
    v[::977] = np.nan
    pos_o, cnt_o, _ = oracle.select_f32(v, 0.5, "lt")
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    knobs = {} if mid is None else {"VD_SEL_MID": mid.split("/")[0]}
    if mid and "/" in mid:  # branching chunks above 100 positions through the fixed lane loop
        knobs["VD_SEL_UNROLL"] = mid.split("/")[1]
    with env(**knobs):
        _density_mix_check(fn, v, n, pos_o, cnt_o)


def _density_mix_check(fn, v, n, pos_o, cnt_o):
    got = _select(fn, torch.from_numpy(v).cuda(), n, 0.5, shift=3)
    assert vd.last_fragment() == "sel_lag"
    assert len(got) == cnt_o and np.array_equal(got, pos_o)
    a = np.where(np.isnan(v), -2**31, np.where(v < 0.5, 1, 9)).astype(np.int32)
    out = torch.empty(n, dtype=torch.int32, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    fn([vd.column(torch.from_numpy(a).cuda())], n, vd.pred([[(0, "<", 5)]]), out_pos=out, out_count=cnt)
    assert vd.last_fragment() == "sel_lag"
    k = int(cnt.item())
    assert k == cnt_o and np.array_equal(out[:k].cpu().numpy(), pos_o)


@pytest.mark.parametrize("mode", ["branch", "predicated"])
@pytest.mark.parametrize("cmp,thr", [("<", -700), (">=", 250), ("==", 17), ("<=", 999)])
def test_lag_select_i32_large_vs_interpreter(mode, cmp, thr):
    """k_sel_lag on an int32 column of 12 M rows (several tiles per CTA, a
    ragged last tile): negative values, epsilon (INT32_MIN, never selected:
    A9), one-sided / equality / nearly-all predicates, against the oracle's
    interpreter (comparison -> FoldSelect)."""
    n = 12 * 10**6 + 777
    rng = np.random.default_rng(4242 + thr)
    a = rng.integers(-1000, 1000, n).astype(np.int32)
    m = rng.random(n) < 0.003
    a[m] = -2**31
    prog = {"<": f"p := Greater({thr}, v)", ">=": f"p := Greater(v, {thr - 1})",
            "==": f"p := Equals(v, {thr})", "<=": f"p := Greater({thr + 1}, v)"}[cmp]
    res = oracle.run(prog + "\npos := FoldSelect(p)", v=(a.astype(np.int64), m))
    pos, pe = res.get_arrays("pos")
    exp = pos[~pe]
    fn = vd.select_branch if mode == "branch" else vd.select_predicated
    out = torch.full((n + 4,), -7, dtype=torch.int32, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    fn([vd.column(torch.from_numpy(a).cuda())], n, vd.pred([[(0, cmp, thr)]]), out_pos=out[1:n + 1], out_count=cnt)
    assert vd.last_fragment() == "sel_lag"
    k = int(cnt.item())
    assert k == exp.size and np.array_equal(out[1:k + 1].cpu().numpy(), exp)
    assert out[0].item() == -7 and (k == n or out[k + 1].item() == -7)


def test_lag_select_in_cuda_graph():
    """k_sel_lag's launch (table memset + cooperative kernel) captured in a
    CUDA graph and replayed: every replay equals the oracle, for two
    thresholds captured in two graphs replayed alternately."""
    n = 20 * 10**6 + 3
    v = gen.host(gen.F32_UNIFORM, n, seed=77)
    dv = torch.from_numpy(v).cuda()
    graphs, outs, exps = [], [], []
    side = torch.cuda.Stream()
    side.wait_stream(torch.cuda.current_stream())
    for t in (0.05, 0.6):
        t = float(np.float32(t))
        pos_o, cnt_o, _ = oracle.select_f32(v, t, "lt")
        exps.append(pos_o)
        out = torch.empty(n, dtype=torch.int32, device="cuda")
        cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
        ws = vd.alloc_ws(vd.workspace_bytes(vd.VD_OP_SELECT, n), dv.device)
        g = torch.cuda.CUDAGraph()
        with torch.cuda.stream(side):
            with torch.cuda.graph(g, stream=side):
                vd.select_branch([vd.column(dv)], n, vd.pred([[(0, "<", t)]]), out_pos=out, out_count=cnt, ws=ws,
                                 stream=side)
        assert vd.last_fragment() == "sel_lag"
        graphs.append(g)
        outs.append((out, cnt, ws))
    torch.cuda.current_stream().wait_stream(side)
    torch.cuda.synchronize()
    for rep in range(3):
        for g, (out, cnt, _), exp in zip(graphs, outs, exps):
            out.fill_(-1)
            cnt.zero_()
            g.replay()
            torch.cuda.synchronize()
            k = int(cnt.item())
            assert k == exp.size and np.array_equal(out[:k].cpu().numpy(), exp), rep
