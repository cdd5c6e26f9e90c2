"""ctypes binding of libvd.so (include/vd.h) -- argument marshalling only.

Every step of the hot path runs in the library's CUDA kernels; this module
only converts torch tensors / Python values into the C ABI's structs and
pointers, allocates workspace through torch (device memory plumbing), and
raises :class:`VdError` on a non-OK status.  There is no CPU fallback: if
``libvd.so`` is missing this module raises at import time, and every compute
call on a machine without a CUDA device fails with ``VD_E_CUDA``.

Names follow the C entry points: ``vd_select_branch`` -> :func:`select_branch`
and so on.  Citations of the paper passages are in include/vd.h.
"""
from __future__ import annotations

import ctypes
import os
from ctypes import POINTER, Structure, c_double, c_int32, c_int64, c_size_t, c_void_p
from typing import Optional, Sequence

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_HERE, "libvd.so")

if not os.path.exists(LIB_PATH):
    raise ImportError(f"{LIB_PATH} is missing: build it with `make` (or __graft_entry__.build()); "
                      "the Voodoo hot path has no CPU fallback")
_L = ctypes.CDLL(LIB_PATH)

# ---- enums (vd.h) -------------------------------------------------------------
VD_OK, VD_E_NULL, VD_E_DTYPE, VD_E_SHAPE, VD_E_CTRL, VD_E_DOMAIN, VD_E_OVERFLOW, VD_E_WORKSPACE, VD_E_CUDA, \
    VD_E_UNSUPPORTED, VD_E_ARG = range(11)
VD_U8, VD_I32, VD_I64, VD_F32, VD_F64 = range(5)
VD_CMP_GT, VD_CMP_LT, VD_CMP_EQ, VD_CMP_GE, VD_CMP_LE, VD_CMP_NE, VD_CMP_IN = range(7)
VD_SEL_BRANCH, VD_SEL_PREDICATED, VD_SEL_PREDICATED_LOOKUP = 0, 1, 2
VD_OP_SELECT, VD_OP_FOLD, VD_OP_SCATTER, VD_OP_PIPELINE, VD_OP_FOLD_SELECT, VD_OP_PARTITION, VD_OP_FOLD_SCAN = range(7)
VD_AGG_SUM, VD_AGG_COUNT, VD_AGG_MIN, VD_AGG_MAX = range(4)
VD_SCATTER_UNIQUE = 1
VD_MAT_NONE, VD_MAT_BREAK, VD_MAT_CHUNKS = 0, 1, 2
VD_COL_NOEPS = 1
VD_MAX_TERMS, VD_MAX_CONJ, VD_MAX_AGGS, VD_MAX_FACTORS, VD_MAX_GATHERS, VD_MAX_KEYPARTS = 8, 4, 8, 3, 4, 3
VD_WS_DOMAIN_ERRORS_OFFSET = 128

EPS_U8 = 0xFF
EPS_I32 = -(2 ** 31)
EPS_I64 = -(2 ** 63)

CMP = {">": VD_CMP_GT, "<": VD_CMP_LT, "==": VD_CMP_EQ, ">=": VD_CMP_GE, "<=": VD_CMP_LE, "!=": VD_CMP_NE,
       "in": VD_CMP_IN}


class vd_column(Structure):
    _fields_ = [("data", c_void_p), ("len", c_int64), ("dtype", c_int32), ("scale", c_int32), ("min", c_int64),
                ("max", c_int64), ("has_minmax", c_int32), ("flags", c_int32)]


class vd_ctrl(Structure):
    _fields_ = [("from_", c_int64), ("step_num", c_int64), ("step_den", c_int64), ("cap", c_int64),
                ("materialized", c_void_p), ("mat_dtype", c_int32), ("reserved", c_int32)]


class vd_term(Structure):
    _fields_ = [("col", c_int32), ("cmp", c_int32), ("ival", c_int64), ("fval", c_double)]


class vd_conj(Structure):
    _fields_ = [("nterms", c_int32), ("reserved", c_int32), ("terms", vd_term * VD_MAX_TERMS)]


class vd_pred(Structure):
    _fields_ = [("nconj", c_int32), ("reserved", c_int32), ("conj", vd_conj * VD_MAX_CONJ)]


class vd_factor(Structure):
    _fields_ = [("col", c_int32), ("reserved", c_int32), ("a", c_int64), ("b", c_int64)]


class vd_agg(Structure):
    _fields_ = [("kind", c_int32), ("nfactors", c_int32), ("f", vd_factor * VD_MAX_FACTORS)]


class vd_keypart(Structure):
    _fields_ = [("col", c_int32), ("fn", c_int32), ("sub", c_int64), ("mult", c_int64)]


class vd_gatherspec(Structure):
    _fields_ = [("fk_col", c_int32), ("dim_col", c_int32), ("bias", c_int64)]


class vd_pipeline(Structure):
    _fields_ = [("pred", vd_pred), ("sel_mode", c_int32), ("ngathers", c_int32),
                ("gathers", vd_gatherspec * VD_MAX_GATHERS), ("nkeyparts", c_int32), ("reserved", c_int32),
                ("key", vd_keypart * VD_MAX_KEYPARTS), ("ngroups", c_int64), ("naggs", c_int32),
                ("force_generic", c_int32), ("aggs", vd_agg * VD_MAX_AGGS), ("materialize", c_int32),
                ("reserved2", c_int32), ("mat_chunk", c_int64)]


class vd_result(Structure):
    _fields_ = [("capacity", c_int64), ("keys", c_void_p), ("aggs", c_void_p), ("rows", c_void_p),
                ("ngroups", c_void_p)]


_P = POINTER
_sigs = {
    "vd_status_str": (ctypes.c_char_p, [c_int32]),
    "vd_last_error": (ctypes.c_char_p, []),
    "vd_version": (ctypes.c_char_p, []),
    "vd_ctrl_runs": (c_int32, [_P(vd_ctrl), c_int64, _P(c_int64)]),
    "vd_workspace_bytes": (c_int32, [c_int32, c_int64, _P(vd_ctrl), _P(vd_pipeline), _P(c_size_t)]),
    "vd_load_column": (c_int32, [c_void_p, c_int64, c_int32, c_int32, c_void_p, c_int32, c_void_p, _P(vd_column)]),
    "vd_select_branch": (c_int32, [_P(vd_column), c_int32, c_int64, _P(vd_pred), _P(vd_ctrl), c_void_p, c_void_p,
                                   c_void_p, c_void_p, c_void_p, c_size_t, c_void_p]),
    "vd_select_predicated": (c_int32, [_P(vd_column), c_int32, c_int64, _P(vd_pred), _P(vd_ctrl), c_void_p,
                                       c_void_p, c_void_p, c_void_p, c_void_p, c_size_t, c_void_p]),
    "vd_fold_select": (c_int32, [_P(vd_column), _P(vd_ctrl), c_int32, c_void_p, c_void_p, c_void_p, c_void_p,
                                 c_void_p, c_size_t, c_void_p]),
    "vd_fold_sum": (c_int32, [_P(vd_column), _P(vd_ctrl), c_void_p, c_void_p, c_void_p, c_void_p, c_size_t,
                              c_void_p]),
    "vd_fold_count": (c_int32, [_P(vd_column), _P(vd_ctrl), c_void_p, c_void_p, c_void_p, c_size_t, c_void_p]),
    "vd_fold_min": (c_int32, [_P(vd_column), _P(vd_ctrl), c_void_p, c_void_p, c_void_p, c_void_p, c_size_t,
                              c_void_p]),
    "vd_fold_max": (c_int32, [_P(vd_column), _P(vd_ctrl), c_void_p, c_void_p, c_void_p, c_void_p, c_size_t,
                              c_void_p]),
    "vd_fold_scan": (c_int32, [_P(vd_column), _P(vd_ctrl), c_void_p, c_void_p, c_size_t, c_void_p]),
    "vd_gather": (c_int32, [_P(vd_column), c_void_p, c_int64, c_int64, c_void_p, c_void_p]),
    "vd_gather_multi": (c_int32, [_P(vd_column), c_int32, c_void_p, c_int64, c_int64, _P(c_void_p), c_void_p]),
    "vd_row_layout": (c_int32, [_P(c_int32), c_int32, _P(c_int32), _P(c_int32)]),
    "vd_zip": (c_int32, [_P(vd_column), c_int32, c_void_p, c_int64, c_void_p]),
    "vd_gather_rows": (c_int32, [c_void_p, c_int64, _P(c_int32), c_int32, c_void_p, c_int64, c_int64, _P(c_void_p),
                                 c_void_p]),
    "vd_scatter": (c_int32, [_P(vd_column), c_void_p, c_int64, c_void_p, c_int64, c_int32, c_void_p, c_size_t,
                             c_void_p]),
    "vd_partition": (c_int32, [_P(vd_column), c_int64, c_int64, c_void_p, c_void_p, c_void_p, c_size_t, c_void_p]),
    "vd_partials_bytes": (c_size_t, [_P(vd_pipeline)]),
    "vd_run_pipeline": (c_int32, [_P(vd_pipeline), _P(vd_column), c_int32, c_int64, _P(vd_column), c_int32,
                                  c_void_p, c_void_p, c_size_t, c_void_p]),
    "vd_merge_partials": (c_int32, [_P(vd_pipeline), _P(vd_column), c_int32, _P(vd_column), c_int32,
                                    _P(c_void_p), c_int32, _P(vd_result)]),
    "vd_merge_partials_device": (c_int32, [_P(vd_pipeline), _P(vd_column), c_int32, _P(vd_column), c_int32,
                                           c_void_p, c_int32, _P(vd_result), c_void_p]),
    "vd_group_fold_ws_bytes": (c_int32, [c_int64, c_int32, _P(c_size_t)]),
    "vd_group_fold": (c_int32, [_P(vd_column), c_int32, c_int64, _P(vd_pred), c_int32, _P(vd_agg), c_int32,
                                c_void_p, c_void_p, c_void_p, c_void_p, c_void_p, c_size_t, c_void_p]),
    "vd_hash_group_fold_ws_bytes": (c_int32, [c_int64, c_int32, _P(c_size_t)]),
    "vd_hash_group_fold": (c_int32, [_P(vd_column), c_int32, c_int64, _P(vd_pred), c_int32, _P(vd_agg), c_int32,
                                     c_int64, c_void_p, c_void_p, c_void_p, c_void_p, c_void_p, c_size_t, c_void_p]),
    "vd_merge_groups_ws_bytes": (c_int32, [c_int64, c_int32, _P(c_size_t)]),
    "vd_merge_groups": (c_int32, [c_void_p, c_void_p, c_void_p, c_void_p, c_int32, c_int64, _P(c_int32), _P(c_int32),
                                  c_int32, c_int64, c_void_p, c_void_p, c_void_p, c_void_p, c_void_p, c_size_t,
                                  c_void_p]),
    "vd_last_launch_count": (c_int32, []),
    "vd_last_fragment": (ctypes.c_char_p, []),
    "vd_abi_struct_sizes": (c_int32, [_P(c_size_t), c_int32]),
}
EXPORTS = sorted(_sigs)
for _name, (_res, _args) in _sigs.items():
    _f = getattr(_L, _name)  # AttributeError if the library lacks a declared symbol
    _f.restype = _res
    _f.argtypes = _args


def _check_abi():
    out = (c_size_t * 9)()
    _L.vd_abi_struct_sizes(out, 9)
    mine = [ctypes.sizeof(t) for t in (vd_column, vd_ctrl, vd_term, vd_conj, vd_pred, vd_agg, vd_keypart,
                                       vd_pipeline, vd_result)]
    if list(out) != mine:
        raise ImportError(f"libvd ABI struct sizes {list(out)} != binding {mine}")


_check_abi()


class VdError(RuntimeError):
    def __init__(self, status: int, where: str):
        self.status = status
        msg = _L.vd_last_error().decode()
        super().__init__(f"{where}: {_L.vd_status_str(status).decode()} {msg}")


def _ok(st: int, where: str):
    if st != VD_OK:
        raise VdError(st, where)


def version() -> str:
    return _L.vd_version().decode()


def last_launch_count() -> int:
    return int(_L.vd_last_launch_count())


def last_fragment() -> str:
    """Name of the fragment the last run_pipeline on this thread ran."""
    return _L.vd_last_fragment().decode()


# ---- torch plumbing ---------------------------------------------------------------
def _torch():
    import torch
    return torch


_TORCH_DT = None


def dtype_of(t) -> int:
    global _TORCH_DT
    torch = _torch()
    if _TORCH_DT is None:
        _TORCH_DT = {torch.uint8: VD_U8, torch.int32: VD_I32, torch.int64: VD_I64, torch.float32: VD_F32,
                     torch.float64: VD_F64}
    try:
        return _TORCH_DT[t.dtype]
    except KeyError:
        raise VdError(VD_E_DTYPE, f"unsupported tensor dtype {t.dtype}") from None


def _ptr(t) -> Optional[int]:
    return None if t is None else t.data_ptr()


def _stream(stream) -> Optional[int]:
    if stream is None:
        torch = _torch()
        return torch.cuda.current_stream().cuda_stream if torch.cuda.is_available() else None
    return stream if isinstance(stream, int) else stream.cuda_stream


def column(t, minmax: Optional[Sequence[int]] = None, scale: int = 0, length: Optional[int] = None,
           noeps: bool = False) -> vd_column:
    """A vd_column view of a contiguous CUDA tensor (no copy).  noeps: the
    caller has verified that no slot is epsilon (sets VD_COL_NOEPS)."""
    if not t.is_contiguous():
        raise VdError(VD_E_SHAPE, "column tensors must be contiguous")
    c = vd_column()
    c.data = t.data_ptr()
    c.len = t.numel() if length is None else length
    c.dtype = dtype_of(t)
    c.scale = scale
    if minmax is not None:
        c.min, c.max = int(minmax[0]), int(minmax[1])
        c.has_minmax = 1
    if noeps:
        c.flags |= VD_COL_NOEPS
    c._keep = t  # the view keeps its tensor alive (the ABI struct holds a raw pointer)
    return c


def column_meta(dtype) -> vd_column:
    """A vd_column carrying only a dtype (vd_dtype int or numpy dtype), no
    data: what vd_merge_partials reads of the views a plan ran with."""
    import numpy as np
    c = vd_column()
    if not isinstance(dtype, int):
        dtype = {np.dtype(np.uint8): VD_U8, np.dtype(np.int32): VD_I32, np.dtype(np.int64): VD_I64,
                 np.dtype(np.float32): VD_F32, np.dtype(np.float64): VD_F64}[np.dtype(dtype)]
    c.dtype = dtype
    return c


def ctrl(from_: int = 0, num: int = 1, den: int = 1, cap: int = 0, materialized=None) -> vd_ctrl:
    """Control vector: virtual (from + floor(i*num/den)) mod cap, or a materialized int32/int64 tensor."""
    c = vd_ctrl()
    c.from_, c.step_num, c.step_den, c.cap = from_, num, den, cap
    if materialized is not None:
        c.materialized = materialized.data_ptr()
        c.mat_dtype = dtype_of(materialized)
        c._keep = materialized
    return c


def pred(conjs: Sequence[Sequence[tuple]]) -> vd_pred:
    """OR of AND-lists of terms (col, op, value); op in > < == >= <= != in.

    ``in`` takes a list of dictionary codes (0..63)."""
    p = vd_pred()
    if len(conjs) > VD_MAX_CONJ:
        raise VdError(VD_E_ARG, "too many conjunctions")
    p.nconj = len(conjs)
    for ci, terms in enumerate(conjs):
        if len(terms) > VD_MAX_TERMS:
            raise VdError(VD_E_ARG, "too many terms")
        p.conj[ci].nterms = len(terms)
        for ti, (col, op, val) in enumerate(terms):
            t = p.conj[ci].terms[ti]
            t.col = col
            t.cmp = CMP[op]
            if op == "in":
                m = 0
                for code in val:
                    m |= 1 << int(code)
                t.ival = m - (1 << 64) if m >= (1 << 63) else m
            elif isinstance(val, float):
                t.fval = val
                t.ival = int(val) if abs(val) < 2 ** 62 else 0
            else:
                t.ival = int(val)
                t.fval = float(val)
    return p


def workspace_bytes(op: int, n: int, ctl: Optional[vd_ctrl] = None, plan: Optional[vd_pipeline] = None) -> int:
    b = c_size_t()
    _ok(_L.vd_workspace_bytes(op, n, ctypes.byref(ctl) if ctl is not None else None,
                              ctypes.byref(plan) if plan is not None else None, ctypes.byref(b)),
        "vd_workspace_bytes")
    return int(b.value)


def alloc_ws(nbytes: int, device=None):
    torch = _torch()
    return torch.empty(max(int(nbytes), 256), dtype=torch.uint8, device=device or "cuda")


def ctrl_runs(ctl: Optional[vd_ctrl], n: int) -> int:
    r = c_int64()
    _ok(_L.vd_ctrl_runs(ctypes.byref(ctl) if ctl is not None else None, n, ctypes.byref(r)), "vd_ctrl_runs")
    return int(r.value)


def _cols_array(cols: Sequence[vd_column]):
    arr = (vd_column * max(1, len(cols)))()
    for i, c in enumerate(cols):
        arr[i] = c
    return arr


# ---- a1 load ---------------------------------------------------------------------------
def load_column(host_src, dev_dst, compute_minmax: bool = True, scale: int = 0, stream=None) -> vd_column:
    """vd_load_column: copy a host array (numpy / CPU tensor) into `dev_dst` (CUDA tensor)."""
    import numpy as np
    torch = _torch()
    if isinstance(host_src, torch.Tensor):
        ptr, n, dt = host_src.data_ptr(), host_src.numel(), dtype_of(host_src)
    else:
        a = np.ascontiguousarray(host_src)
        ptr, n = a.ctypes.data, a.size
        dt = {np.dtype(np.uint8): VD_U8, np.dtype(np.int32): VD_I32, np.dtype(np.int64): VD_I64,
              np.dtype(np.float32): VD_F32, np.dtype(np.float64): VD_F64}[a.dtype]
        host_src = a
    out = vd_column()
    _ok(_L.vd_load_column(ptr, n, dt, scale, dev_dst.data_ptr(), int(compute_minmax), _stream(stream),
                          ctypes.byref(out)), "vd_load_column")
    return out


# ---- a2+a3 selection ---------------------------------------------------------------------
def _select(fn, name, cols, n, p, ctl, out_pos, out_count, out_run_off, out_nruns, ws, stream):
    arr = _cols_array(cols)
    if ws is None:
        ws = alloc_ws(workspace_bytes(VD_OP_SELECT, n, ctl), out_count.device)
    _ok(fn(arr, len(cols), n, ctypes.byref(p) if p is not None else None,
           ctypes.byref(ctl) if ctl is not None else None, _ptr(out_pos), _ptr(out_count), _ptr(out_run_off),
           _ptr(out_nruns), ws.data_ptr(), ws.numel(), _stream(stream)), name)


def select_branch(cols, n, p, ctl=None, *, out_pos, out_count, out_run_off=None, out_nruns=None, ws=None,
                  stream=None):
    _select(_L.vd_select_branch, "vd_select_branch", cols, n, p, ctl, out_pos, out_count, out_run_off, out_nruns,
            ws, stream)


def select_predicated(cols, n, p, ctl=None, *, out_pos, out_count, out_run_off=None, out_nruns=None, ws=None,
                      stream=None):
    _select(_L.vd_select_predicated, "vd_select_predicated", cols, n, p, ctl, out_pos, out_count, out_run_off,
            out_nruns, ws, stream)


# ---- a6 folds -------------------------------------------------------------------------------
def fold_select(s: vd_column, ctl=None, sel_mode=VD_SEL_BRANCH, *, out_pos, out_count, out_run_off=None,
                out_nruns=None, ws=None, stream=None):
    if ws is None:
        ws = alloc_ws(workspace_bytes(VD_OP_FOLD_SELECT, s.len, ctl), out_count.device)
    _ok(_L.vd_fold_select(ctypes.byref(s), ctypes.byref(ctl) if ctl is not None else None, sel_mode, _ptr(out_pos),
                          _ptr(out_count), _ptr(out_run_off), _ptr(out_nruns), ws.data_ptr(), ws.numel(),
                          _stream(stream)), "vd_fold_select")


def _fold(fn, name, vals, ctl, out, out_counts, out_nruns, ws, stream, has_counts=True):
    if ws is None:
        ws = alloc_ws(workspace_bytes(VD_OP_FOLD, vals.len, ctl), out.device if out is not None else None)
    c = ctypes.byref(ctl) if ctl is not None else None
    if has_counts:
        st = fn(ctypes.byref(vals), c, _ptr(out), _ptr(out_counts), _ptr(out_nruns), ws.data_ptr(), ws.numel(),
                _stream(stream))
    else:
        st = fn(ctypes.byref(vals), c, _ptr(out), _ptr(out_nruns), ws.data_ptr(), ws.numel(), _stream(stream))
    _ok(st, name)


def fold_sum(vals, ctl=None, *, out, out_counts=None, out_nruns=None, ws=None, stream=None):
    _fold(_L.vd_fold_sum, "vd_fold_sum", vals, ctl, out, out_counts, out_nruns, ws, stream)


def fold_count(vals, ctl=None, *, out, out_nruns=None, ws=None, stream=None):
    _fold(_L.vd_fold_count, "vd_fold_count", vals, ctl, out, None, out_nruns, ws, stream, has_counts=False)


def fold_min(vals, ctl=None, *, out, out_counts=None, out_nruns=None, ws=None, stream=None):
    _fold(_L.vd_fold_min, "vd_fold_min", vals, ctl, out, out_counts, out_nruns, ws, stream)


def fold_max(vals, ctl=None, *, out, out_counts=None, out_nruns=None, ws=None, stream=None):
    _fold(_L.vd_fold_max, "vd_fold_max", vals, ctl, out, out_counts, out_nruns, ws, stream)


def fold_scan(vals, ctl=None, *, out, ws=None, stream=None):
    """vd_fold_scan: per-run inclusive prefix sums into `out` (int64 or
    float64 CUDA tensor of vals.len slots)."""
    if ws is None:
        ws = alloc_ws(workspace_bytes(VD_OP_FOLD_SCAN, vals.len, ctl), out.device)
    c = ctypes.byref(ctl) if ctl is not None else None
    _ok(_L.vd_fold_scan(ctypes.byref(vals), c, _ptr(out), ws.data_ptr(), ws.numel(), _stream(stream)),
        "vd_fold_scan")


def describe(t, scale: int = 0, stream=None) -> vd_column:
    """a1 metadata for a device-resident column: min / max of
    the non-epsilon values and VD_COL_NOEPS, computed on the device by the
    library's own FoldMin / FoldMax (their per-run non-epsilon counts tell
    whether any slot is epsilon).  Float columns get no metadata."""
    import torch
    c = column(t, scale=scale)
    if c.dtype in (VD_F32, VD_F64) or t.numel() == 0:
        return c
    lo = torch.empty(1, dtype=t.dtype, device=t.device)
    hi = torch.empty(1, dtype=t.dtype, device=t.device)
    cnt = torch.empty(1, dtype=torch.int64, device=t.device)
    fold_min(c, None, out=lo, out_counts=cnt, stream=stream)
    fold_max(c, None, out=hi, stream=stream)
    k = int(cnt.item())
    if k == 0:
        return c
    return column(t, minmax=(int(lo.item()), int(hi.item())), scale=scale, noeps=(k == t.numel()))


# ---- a4 gather / a5 scatter, partition -------------------------------------------------------
def gather(src: vd_column, pos, n, bias, out, stream=None):
    _ok(_L.vd_gather(ctypes.byref(src), _ptr(pos), n, bias, _ptr(out), _stream(stream)), "vd_gather")


def gather_multi(srcs: Sequence[vd_column], pos, n, bias, outs, stream=None):
    arr = _cols_array(srcs)
    o = (c_void_p * len(outs))(*[t.data_ptr() for t in outs])
    _ok(_L.vd_gather_multi(arr, len(srcs), _ptr(pos), n, bias, o, _stream(stream)), "vd_gather_multi")


def row_layout(dtypes: Sequence[int]):
    """vd_row_layout: (field offsets, row stride) of the row-wise format (Fig 14 Layout Transform)."""
    k = len(dtypes)
    dt = (c_int32 * k)(*dtypes)
    offs = (c_int32 * k)()
    st = c_int32()
    _ok(_L.vd_row_layout(dt, k, offs, ctypes.byref(st)), "vd_row_layout")
    return list(offs), st.value


def zip_rows(cols: Sequence[vd_column], out_rows, stream=None):
    """vd_zip: materialise the columns row-wise into `out_rows` (CUDA uint8 tensor, len*stride bytes)."""
    arr = _cols_array(cols)
    _ok(_L.vd_zip(arr, len(cols), _ptr(out_rows), out_rows.numel() * out_rows.element_size(), _stream(stream)),
        "vd_zip")


def gather_rows(rows, nrows, dtypes: Sequence[int], pos, n, bias, outs, stream=None):
    """vd_gather_rows: resolve positions into the row-wise table, field k -> outs[k]."""
    k = len(dtypes)
    dt = (c_int32 * k)(*dtypes)
    o = (c_void_p * k)(*[t.data_ptr() for t in outs])
    _ok(_L.vd_gather_rows(_ptr(rows), nrows, dt, k, _ptr(pos), n, bias, o, _stream(stream)), "vd_gather_rows")


def scatter(src: vd_column, pos, n, out, out_len, unique=False, ws=None, stream=None):
    if ws is None and not unique:
        ws = alloc_ws(workspace_bytes(VD_OP_SCATTER, out_len), out.device)
    _ok(_L.vd_scatter(ctypes.byref(src), _ptr(pos), n, _ptr(out), out_len, VD_SCATTER_UNIQUE if unique else 0,
                      _ptr(ws), ws.numel() if ws is not None else 0, _stream(stream)), "vd_scatter")


def partition(v: vd_column, pivot_from, npivots, out_pos, out_bucket_counts=None, ws=None, stream=None):
    if ws is None:
        ws = alloc_ws(workspace_bytes(VD_OP_PARTITION, v.len), out_pos.device)
    _ok(_L.vd_partition(ctypes.byref(v), pivot_from, npivots, _ptr(out_pos), _ptr(out_bucket_counts),
                        ws.data_ptr(), ws.numel(), _stream(stream)), "vd_partition")


# ---- a7-a9 fused pipeline ----------------------------------------------------------------------
def pipeline(*, pred_: Optional[vd_pred] = None, sel_mode: int = VD_SEL_BRANCH, gathers=(), key=(), ngroups=1,
             aggs=(), force_generic=False, materialize: int = VD_MAT_NONE, mat_chunk: int = 0) -> vd_pipeline:
    """Build a vd_pipeline.

    materialize: VD_MAT_NONE (fused), VD_MAT_BREAK (the predicate
    materialised, Fig 8's break) or VD_MAT_CHUNKS (per-chunk position lists
    of mat_chunk rows, Fig 15's vectorized plan).

    gathers: [(fk_col, dim_col, bias)]; key: [(col, fn, sub, mult)] (fn 0 identity, 1 year);
    aggs: [("sum", [(col, a, b), ...]) | ("count",) | ("min", [...]) | ("max", [...])], factor = a + b*col
    (col -1: constant a).  A bare int factor c means the plain column (c, 0, 1).
    """
    p = vd_pipeline()
    if pred_ is not None:
        p.pred = pred_
    p.sel_mode = sel_mode
    p.ngathers = len(gathers)
    for i, (fk, dc, bias) in enumerate(gathers):
        p.gathers[i].fk_col, p.gathers[i].dim_col, p.gathers[i].bias = fk, dc, bias
    p.nkeyparts = len(key)
    for i, (col, fn, sub, mult) in enumerate(key):
        p.key[i].col, p.key[i].fn, p.key[i].sub, p.key[i].mult = col, fn, sub, mult
    p.ngroups = ngroups
    p.naggs = len(aggs)
    kinds = {"sum": VD_AGG_SUM, "count": VD_AGG_COUNT, "min": VD_AGG_MIN, "max": VD_AGG_MAX}
    for i, ag in enumerate(aggs):
        p.aggs[i].kind = kinds[ag[0]]
        facs = ag[1] if len(ag) > 1 else []
        p.aggs[i].nfactors = len(facs)
        for j, f in enumerate(facs):
            if isinstance(f, int):
                f = (f, 0, 1)
            p.aggs[i].f[j].col, p.aggs[i].f[j].a, p.aggs[i].f[j].b = f
    p.force_generic = int(force_generic)
    p.materialize = int(materialize)
    p.mat_chunk = int(mat_chunk)
    return p


def aggs_array(aggs):
    """A ctypes vd_agg[] from the pipeline() aggregate notation."""
    return (vd_agg * max(1, len(aggs)))(*pipeline(aggs=aggs).aggs[:max(1, len(aggs))]) if aggs else None


def group_fold_ws_bytes(domain: int, naggs: int) -> int:
    b = c_size_t(0)
    _ok(_L.vd_group_fold_ws_bytes(domain, naggs, ctypes.byref(b)), "vd_group_fold_ws_bytes")
    return int(b.value)


def group_fold(cols: Sequence[vd_column], n: int, key_col: int, aggs=(), pred_: Optional[vd_pred] = None, *,
               out_keys, out_aggs, out_rows, out_ngroups, ws=None, stream=None):
    """vd_group_fold (NEXT-4): grouped fold over the key column's min/max
    domain; outputs are CUDA tensors (int64 keys / rows / ngroups[1], uint8
    aggregate slots of 16 bytes x naggs per group)."""
    k = cols[key_col]
    if ws is None:
        if not k.has_minmax:
            raise VdError(VD_E_DOMAIN, "group_fold: key column without min/max")
        ws = alloc_ws(group_fold_ws_bytes(k.max - k.min + 1, len(aggs)), out_keys.device)
    arr = _cols_array(cols)
    ag = aggs_array(aggs)
    _ok(_L.vd_group_fold(arr, len(cols), n, ctypes.byref(pred_) if pred_ is not None else None, key_col, ag,
                         len(aggs), out_keys.data_ptr(), _ptr(out_aggs), out_rows.data_ptr(), out_ngroups.data_ptr(),
                         ws.data_ptr(), ws.numel(), _stream(stream)), "vd_group_fold")


def hash_group_fold_ws_bytes(max_groups: int, naggs: int) -> int:
    b = c_size_t(0)
    _ok(_L.vd_hash_group_fold_ws_bytes(max_groups, naggs, ctypes.byref(b)), "vd_hash_group_fold_ws_bytes")
    return int(b.value)


def merge_groups_ws_bytes(max_groups: int, naggs: int) -> int:
    b = c_size_t(0)
    _ok(_L.vd_merge_groups_ws_bytes(max_groups, naggs, ctypes.byref(b)), "vd_merge_groups_ws_bytes")
    return int(b.value)


def hash_group_fold(cols: Sequence[vd_column], n: int, key_col: int, aggs=(), pred_: Optional[vd_pred] = None, *,
                    max_groups: int, out_keys, out_aggs, out_rows, out_ngroups, ws=None, stream=None):
    """vd_hash_group_fold (NEXT-4, sparse keys): open-addressing table sized
    from max_groups (an upper bound on the distinct keys); groups come out in
    table order; out_ngroups[0] = -1 if the table filled up."""
    if ws is None:
        ws = alloc_ws(hash_group_fold_ws_bytes(max_groups, len(aggs)), out_keys.device)
    arr = _cols_array(cols)
    ag = aggs_array(aggs)
    _ok(_L.vd_hash_group_fold(arr, len(cols), n, ctypes.byref(pred_) if pred_ is not None else None, key_col, ag,
                              len(aggs), max_groups, out_keys.data_ptr(), _ptr(out_aggs), out_rows.data_ptr(),
                              out_ngroups.data_ptr(), ws.data_ptr(), ws.numel(), _stream(stream)),
        "vd_hash_group_fold")


def merge_groups(keys, aggs_slots, rows, counts, nparts: int, stride: int, kinds: Sequence[int],
                 float_aggs: Sequence[bool], *, max_groups: int, out_keys, out_aggs, out_rows, out_ngroups, ws=None,
                 stream=None):
    """vd_merge_groups: the cross-GPU merge of compacted groups -- nparts
    blocks of `stride` groups (device tensors in the vd_group_fold layout,
    e.g. an all-gather of every rank's padded output), block r holding
    counts[r] (device int64 tensor) valid groups."""
    na = len(kinds)
    if ws is None:
        ws = alloc_ws(merge_groups_ws_bytes(max_groups, na), out_keys.device)
    k = (c_int32 * max(1, na))(*kinds)
    f = (c_int32 * max(1, na))(*[int(bool(x)) for x in float_aggs] + [0] * (na - len(float_aggs)))
    _ok(_L.vd_merge_groups(_ptr(keys), _ptr(aggs_slots), _ptr(rows), _ptr(counts), nparts, stride, k, f, na,
                           max_groups, out_keys.data_ptr(), _ptr(out_aggs), out_rows.data_ptr(),
                           out_ngroups.data_ptr(), ws.data_ptr(), ws.numel(), _stream(stream)), "vd_merge_groups")


def decode_group_slots(buf: bytes, ngroups: int, naggs: int, float_aggs: Sequence[bool] = ()):
    """[[agg values] per group] from vd_group_fold's 16-byte slots."""
    import struct
    out = []
    for g in range(ngroups):
        vals = []
        for a in range(naggs):
            off = (g * naggs + a) * 16
            if a < len(float_aggs) and float_aggs[a]:
                vals.append(struct.unpack_from("<d", buf, off)[0])
            else:
                lo, hi = struct.unpack_from("<Qq", buf, off)
                vals.append(hi * (1 << 64) + lo)
        out.append(vals)
    return out


def partials_bytes(plan: vd_pipeline) -> int:
    return int(_L.vd_partials_bytes(ctypes.byref(plan)))


def run_pipeline(plan: vd_pipeline, cols: Sequence[vd_column], n: int, dims: Sequence[vd_column] = (), *, out,
                 ws=None, stream=None):
    """vd_run_pipeline into `out` (a CUDA uint8 tensor of partials_bytes(plan) bytes)."""
    if ws is None:
        ws = alloc_ws(workspace_bytes(VD_OP_PIPELINE, n, None, plan), out.device)
    arr = _cols_array(cols)
    darr = _cols_array(dims)
    _ok(_L.vd_run_pipeline(ctypes.byref(plan), arr, len(cols), n, darr if len(dims) else None, len(dims),
                           out.data_ptr(), ws.data_ptr(), ws.numel(), _stream(stream)), "vd_run_pipeline")


class HostResult:
    """Host buffers of a vd_result (capacity = plan.ngroups groups)."""

    def __init__(self, plan: vd_pipeline):
        cap = int(plan.ngroups)
        self.naggs = int(plan.naggs)
        self.keys = (ctypes.c_int64 * cap)()
        self.aggs = ctypes.create_string_buffer(max(1, cap * self.naggs * 16))
        self.rows = (ctypes.c_int64 * cap)()
        self.ngroups = ctypes.c_int64(0)
        self.struct = vd_result(cap, ctypes.addressof(self.keys), ctypes.addressof(self.aggs),
                                ctypes.addressof(self.rows), ctypes.addressof(self.ngroups))

    def decode(self, plan: vd_pipeline, float_aggs: Sequence[bool] = ()):
        g = int(self.ngroups.value)
        return decode_result(bytes(self.keys)[:8 * g], self.aggs.raw[:16 * g * self.naggs], bytes(self.rows)[:8 * g],
                             g, plan, float_aggs)


class DeviceResult:
    """Device buffers of a vd_result (torch CUDA tensors)."""

    def __init__(self, plan: vd_pipeline, device=None):
        torch = _torch()
        cap = int(plan.ngroups)
        self.naggs = int(plan.naggs)
        self.keys = torch.empty(cap, dtype=torch.int64, device=device or "cuda")
        self.aggs = torch.empty(max(1, cap * self.naggs * 16), dtype=torch.uint8, device=self.keys.device)
        self.rows = torch.empty(cap, dtype=torch.int64, device=self.keys.device)
        self.ngroups = torch.zeros(1, dtype=torch.int64, device=self.keys.device)
        self.struct = vd_result(cap, self.keys.data_ptr(), self.aggs.data_ptr(), self.rows.data_ptr(),
                                self.ngroups.data_ptr())

    def decode(self, plan: vd_pipeline, float_aggs: Sequence[bool] = ()):
        """Copy the written groups to the host and decode them (synchronises)."""
        g = int(self.ngroups.item())
        return decode_result(self.keys[:g].cpu().numpy().tobytes(),
                             self.aggs[:16 * g * self.naggs].cpu().numpy().tobytes(),
                             self.rows[:g].cpu().numpy().tobytes(), g, plan, float_aggs)


def merge_partials(plan: vd_pipeline, cols: Sequence[vd_column], dims: Sequence[vd_column], parts_host,
                   float_aggs: Sequence[bool] = ()):
    """vd_merge_partials over host byte buffers (rank order): the merged,
    compacted result decoded as {group: [agg values..., row_count]}."""
    nb = partials_bytes(plan)
    bufs = [ctypes.create_string_buffer(bytes(b), nb) for b in parts_host]
    ptrs = (c_void_p * max(1, len(bufs)))(*[ctypes.addressof(b) for b in bufs])
    res = HostResult(plan)
    _ok(_L.vd_merge_partials(ctypes.byref(plan), _cols_array(cols) if cols else None, len(cols),
                             _cols_array(dims) if dims else None, len(dims), ptrs, len(bufs), ctypes.byref(res.struct)),
        "vd_merge_partials")
    return res.decode(plan, float_aggs)


def merge_partials_device(plan: vd_pipeline, cols: Sequence[vd_column], dims: Sequence[vd_column], parts_dev,
                          nparts: int, result: Optional[DeviceResult] = None, stream=None) -> DeviceResult:
    """vd_merge_partials_device: rank-order merge of `nparts` partials held
    back to back in the CUDA tensor `parts_dev`, compacted into `result`
    (allocated if None) on `stream`; nothing synchronises."""
    if result is None:
        result = DeviceResult(plan, parts_dev.device)
    _ok(_L.vd_merge_partials_device(ctypes.byref(plan), _cols_array(cols) if cols else None, len(cols),
                                    _cols_array(dims) if dims else None, len(dims), parts_dev.data_ptr(), nparts,
                                    ctypes.byref(result.struct), _stream(stream)), "vd_merge_partials_device")
    return result


def decode_result(keys: bytes, aggs: bytes, rows: bytes, ngroups: int, plan: vd_pipeline,
                  float_aggs: Sequence[bool] = ()):
    """Byte decoding of a vd_result's first `ngroups` groups (no filtering,
    no arithmetic: the library did the compaction): {key: [agg values...,
    row_count]} in the library's order; integer slots as exact Python ints,
    slots flagged in float_aggs as f64."""
    import struct
    na = int(plan.naggs)
    res = {}
    for j in range(ngroups):
        (k,) = struct.unpack_from("<q", keys, 8 * j)
        (r,) = struct.unpack_from("<q", rows, 8 * j)
        vals = []
        for a in range(na):
            off = (j * na + a) * 16
            if a < len(float_aggs) and float_aggs[a] and plan.aggs[a].kind != VD_AGG_COUNT:
                vals.append(struct.unpack_from("<d", aggs, off)[0])
            else:
                lo, hi = struct.unpack_from("<Qq", aggs, off)
                vals.append(hi * (1 << 64) + lo)
        vals.append(r)
        res[k] = vals
    return res


def decode_partials(buf: bytes, plan: vd_pipeline, float_aggs: Sequence[bool] = ()):
    """{group: [agg values..., row_count]} of ONE device's partials (copied
    to the host): the library's vd_merge_partials with nparts = 1 does the
    Fig 11 compaction (empty groups dropped, ascending key); this function
    only decodes the bytes."""
    return merge_partials(plan, [], [], [buf], float_aggs)
