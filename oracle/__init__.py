"""CPU oracle for the Voodoo hot path -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this package.  The
product path (``paper_journals_pvldb_pirkmzm16_b200``) never does, and the
two share no code (only the seeded input generator in ``gen/``).

Layer 1 -- :class:`Program`: a literal interpreter of Voodoo programs
(§2.2 Table 2) over epsilon-padded vectors, every
intermediate materialised (the paper's interpreter).

Layer 2 -- :func:`q1`, :func:`q6`, :func:`q15`, :func:`select_f32`, :func:`fkj`:
brute-force SQL-equivalent loops (TPC-H SQL [ext]) written independently of
layer 1.  Both layers are plain single-threaded C++17 (``liboracle.so``).

Pins (tests/test_oracle_*.py, run with ``-m "not gpu"``): the worked examples
of Fig 7, Fig 9 and Fig 11 (tests/golden/), the invariants of Fig 1 and
Fig 3/4, closed forms, pandas/numpy special cases and brute force.
"""
from __future__ import annotations

import ctypes
import os
from typing import Dict, Optional

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB = None

EPS = None  # marker used in expected lists for the empty value epsilon

c_i64p = ctypes.POINTER(ctypes.c_int64)


def _lib():
    global _LIB
    if _LIB is None:
        path = os.path.join(_HERE, "liboracle.so")
        if not os.path.exists(path):
            raise RuntimeError(f"{path} missing: run `make`")
        L = ctypes.CDLL(path)
        vp, i64, c = ctypes.c_void_p, ctypes.c_int64, ctypes.c_char_p
        L.or_ctx_new.restype = vp
        L.or_ctx_free.argtypes = [vp]
        L.or_ctx_set_i64.argtypes = [vp, c, vp, vp, i64]
        L.or_ctx_set_f64.argtypes = [vp, c, vp, vp, i64]
        L.or_ctx_run.argtypes = [vp, c, ctypes.c_char_p, ctypes.c_int]
        L.or_ctx_len.argtypes = [vp, c]
        L.or_ctx_len.restype = i64
        L.or_ctx_is_float.argtypes = [vp, c]
        L.or_ctx_get_i128.argtypes = [vp, c, vp, vp, vp]
        L.or_ctx_get_f64.argtypes = [vp, c, vp, vp, vp]
        L.or_q1.argtypes = [i64, vp, vp, vp, vp, vp, vp, vp, ctypes.c_int32, vp, vp]
        L.or_q6.argtypes = [i64, vp, vp, vp, vp, ctypes.c_int32, ctypes.c_int32, i64, i64, i64, vp, vp, vp]
        L.or_q15.argtypes = [i64, vp, vp, vp, vp, ctypes.c_int32, ctypes.c_int32, vp, vp, vp, vp]
        L.or_q15.restype = i64
        L.or_select_f32.argtypes = [i64, vp, ctypes.c_float, ctypes.c_int, vp, vp, vp]
        L.or_select_f32.restype = i64
        L.or_fkj.argtypes = [ctypes.c_int, i64] + [vp] * 8 + [i64, vp, vp, vp, i64, vp, vp, vp]
        L.or_year_of_day.argtypes = [ctypes.c_int32]
        L.or_year_of_day.restype = ctypes.c_int32
        _LIB = L
    return _LIB


def _p(a: Optional[np.ndarray]):
    return None if a is None else a.ctypes.data


class Program:
    """Literal interpreter context: bind inputs, run program text, read results.

    Results are Python lists with ``None`` for epsilon; integers are exact
    Python ints (128-bit in the oracle), floats are Python floats (the long
    double rounded to double; :meth:`get_float_exact` adds the residual).
    """

    def __init__(self):
        self._L = _lib()
        self._ctx = self._L.or_ctx_new()

    def __del__(self):
        try:
            self._L.or_ctx_free(self._ctx)
        except Exception:
            pass

    def set(self, name: str, values, eps=None):
        arr = np.asarray(values)
        e = None
        if eps is not None:
            e = np.ascontiguousarray(np.asarray(eps, dtype=np.uint8))
        if arr.dtype.kind == "f":
            a = np.ascontiguousarray(arr, dtype=np.float64)
            rc = self._L.or_ctx_set_f64(self._ctx, name.encode(), _p(a), _p(e), a.size)
        else:
            a = np.ascontiguousarray(arr, dtype=np.int64)
            rc = self._L.or_ctx_set_i64(self._ctx, name.encode(), _p(a), _p(e), a.size)
        if rc != 0:
            raise ValueError(f"binding {name}: length mismatch with sibling attributes")
        return self

    def run(self, program: str):
        buf = ctypes.create_string_buffer(1024)
        rc = self._L.or_ctx_run(self._ctx, program.encode(), buf, 1024)
        if rc != 0:
            raise RuntimeError(f"oracle program failed: {buf.value.decode()}")
        return self

    def length(self, name: str) -> int:
        return int(self._L.or_ctx_len(self._ctx, name.encode()))

    def is_float(self, name: str) -> bool:
        r = self._L.or_ctx_is_float(self._ctx, name.encode())
        if r < 0:
            raise KeyError(name)
        return bool(r)

    def get_arrays(self, name: str):
        """(values, eps) as numpy arrays; ints are returned as int64 when they fit,
        else as an object array of Python ints."""
        n = self.length(name)
        if n < 0:
            raise KeyError(name)
        eps = np.zeros(n, dtype=np.uint8)
        if self.is_float(name):
            v = np.zeros(n, dtype=np.float64)
            self._L.or_ctx_get_f64(self._ctx, name.encode(), _p(v), None, _p(eps))
            return v, eps.astype(bool)
        lo = np.zeros(n, dtype=np.int64)
        hi = np.zeros(n, dtype=np.int64)
        self._L.or_ctx_get_i128(self._ctx, name.encode(), _p(lo), _p(hi), _p(eps))
        fits = ((hi == 0) & (lo >= 0)) | ((hi == -1) & (lo < 0))
        if fits.all():
            return lo, eps.astype(bool)
        vals = np.array([int(h) * (1 << 64) + (int(l_) & 0xFFFFFFFFFFFFFFFF) for l_, h in zip(lo, hi)],
                        dtype=object)
        return vals, eps.astype(bool)

    def get(self, name: str):
        v, e = self.get_arrays(name)
        out = []
        for x, em in zip(v.tolist(), e.tolist()):
            out.append(None if em else x)
        return out

    def get_float_exact(self, name: str):
        n = self.length(name)
        v = np.zeros(n)
        r = np.zeros(n)
        eps = np.zeros(n, dtype=np.uint8)
        self._L.or_ctx_get_f64(self._ctx, name.encode(), _p(v), _p(r), _p(eps))
        return v, r, eps.astype(bool)


def run(program: str, **inputs) -> Program:
    """Bind keyword inputs (name -> array, or (array, eps)) and run `program`."""
    p = Program()
    for k, v in inputs.items():
        if isinstance(v, tuple):
            p.set(k.replace("__", "."), v[0], v[1])
        else:
            p.set(k.replace("__", "."), v)
    return p.run(program)


def _to_int(lo, hi) -> int:
    return int(hi) * (1 << 64) + (int(lo) & 0xFFFFFFFFFFFFFFFF)


Q1_AGGS = ["sum_qty", "sum_base_price", "sum_disc_price", "sum_charge", "sum_disc", "count"]


def q1(cols: Dict[str, np.ndarray], ship_max: int = 10471):
    """Brute-force TPC-H Q1: {slot k = rf*2+ls: [6 exact ints]} for non-empty slots."""
    n = len(cols["l_shipdate"])
    lo = np.zeros(36, dtype=np.int64)
    hi = np.zeros(36, dtype=np.int64)
    a = {k: np.ascontiguousarray(v) for k, v in cols.items()}
    _lib().or_q1(n, _p(a["l_shipdate"]), _p(a["l_returnflag"]), _p(a["l_linestatus"]), _p(a["l_quantity"]),
                 _p(a["l_extendedprice"]), _p(a["l_discount"]), _p(a["l_tax"]), int(ship_max), _p(lo), _p(hi))
    res = {}
    for k in range(6):
        vals = [_to_int(lo[k * 6 + j], hi[k * 6 + j]) for j in range(6)]
        if vals[5] > 0:
            res[k] = vals
    return res


def q6(cols: Dict[str, np.ndarray], d0: int = 8766, d1: int = 9131, dlo: int = 5, dhi: int = 7,
       qmax: int = 2400):
    """Brute-force TPC-H Q6: (revenue scale 1e4 exact int, count)."""
    n = len(cols["l_shipdate"])
    lo = np.zeros(1, dtype=np.int64)
    hi = np.zeros(1, dtype=np.int64)
    cnt = np.zeros(1, dtype=np.int64)
    a = {k: np.ascontiguousarray(v) for k, v in cols.items()}
    _lib().or_q6(n, _p(a["l_shipdate"]), _p(a["l_discount"]), _p(a["l_quantity"]), _p(a["l_extendedprice"]),
                 int(d0), int(d1), int(dlo), int(dhi), int(qmax), _p(lo), _p(hi), _p(cnt))
    return _to_int(lo[0], hi[0]), int(cnt[0])


def q15(cols: Dict[str, np.ndarray], d0: int = 9496, d1: int = 9587):
    """Brute-force TPC-H Q15 revenue view: {suppkey: (revenue exact int scale 1e4, count)}
    for ship in [d0, d1) (default [1996-01-01, 1996-04-01))."""
    n = len(cols["l_shipdate"])
    key = np.zeros(max(n, 1), dtype=np.int64)
    lo = np.zeros(max(n, 1), dtype=np.int64)
    hi = np.zeros(max(n, 1), dtype=np.int64)
    cnt = np.zeros(max(n, 1), dtype=np.int64)
    a = {k: np.ascontiguousarray(cols[k]) for k in ("l_shipdate", "l_suppkey", "l_extendedprice", "l_discount")}
    g = _lib().or_q15(n, _p(a["l_shipdate"]), _p(a["l_suppkey"]), _p(a["l_extendedprice"]), _p(a["l_discount"]),
                      int(d0), int(d1), _p(key), _p(lo), _p(hi), _p(cnt))
    return {int(key[j]): (_to_int(lo[j], hi[j]), int(cnt[j])) for j in range(g)}


def select_f32(v: np.ndarray, t: float, op: str = "lt", want_positions: bool = True):
    """Brute-force selection (Fig 1): (positions int32, count, long-double sum as (hi, lo))."""
    v = np.ascontiguousarray(v, dtype=np.float32)
    pos = np.empty(v.size, dtype=np.int32) if want_positions else None
    sh = np.zeros(1)
    sl = np.zeros(1)
    c = _lib().or_select_f32(v.size, _p(v), ctypes.c_float(t), 0 if op == "lt" else 1, _p(pos), _p(sh), _p(sl))
    return (pos[:c] if pos is not None else None), int(c), (float(sh[0]), float(sl[0]))


def fkj(variant: int, li: Dict[str, np.ndarray], part: Dict[str, np.ndarray], supp: Dict[str, np.ndarray]):
    """Brute-force FK gather join: {group: (revenue exact int scale 1e4, count)} for non-empty groups."""
    n = len(li["l_partkey"])
    lo = np.zeros(350, dtype=np.int64)
    hi = np.zeros(350, dtype=np.int64)
    a = {k: np.ascontiguousarray(v) for k, v in li.items()}
    p = {k: np.ascontiguousarray(v) for k, v in part.items()}
    s = {k: np.ascontiguousarray(v) for k, v in supp.items()}
    _lib().or_fkj(int(variant), n, _p(a["l_partkey"]), _p(a["l_suppkey"]), _p(a["l_quantity"]),
                  _p(a["l_extendedprice"]), _p(a["l_discount"]), _p(a["l_shipmode"]), _p(a["l_shipinstruct"]),
                  _p(a["l_shipdate"]), len(p["p_brand"]), _p(p["p_brand"]), _p(p["p_container"]), _p(p["p_size"]),
                  len(s["s_nationkey"]), _p(s["s_nationkey"]), _p(lo), _p(hi))
    res = {}
    for g in range(175):
        r = _to_int(lo[2 * g], hi[2 * g])
        c = _to_int(lo[2 * g + 1], hi[2 * g + 1])
        if c > 0:
            res[g] = (r, c)
    return res


def year_of_day(day: int) -> int:
    return int(_lib().or_year_of_day(int(day)))
