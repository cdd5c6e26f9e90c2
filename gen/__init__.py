"""Seeded synthetic inputs shared by the oracle side and the CUDA side.

Thin ctypes binding of ``gen/libvdgen.so`` (built from ``gen/vd_gen.h``).
This module holds none of the Voodoo method's arithmetic -- only random
draws and the dbgen-shaped value recipes.

* :func:`host` fills a numpy array (used to feed the oracle).
* :func:`device` fills a CUDA buffer in place (used to feed the CUDA path at
  full size without a host round trip).

Both produce bit-identical values for the same (column, seed, sf, rows).
"""
from __future__ import annotations

import ctypes
import os

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB = None

# Column ids (gen/vd_gen.h)
L_SHIPDATE = 1
L_RETURNFLAG = 2
L_LINESTATUS = 3
L_QUANTITY = 4
L_EXTENDEDPRICE = 5
L_DISCOUNT = 6
L_TAX = 7
L_PARTKEY = 8
L_SUPPKEY = 9
L_SHIPMODE = 10
L_SHIPINSTRUCT = 11
P_BRAND = 12
P_CONTAINER = 13
P_SIZE = 14
S_NATIONKEY = 15
F32_UNIFORM = 16
I32_UNIFORM = 17
I32_PERM = 18
I64_UNIFORM = 19
F64_UNIFORM = 20

DEFAULT_SEED = 0x5EEDC0DE

_DTYPES = {
    L_SHIPDATE: np.int32, L_RETURNFLAG: np.uint8, L_LINESTATUS: np.uint8, L_QUANTITY: np.int64,
    L_EXTENDEDPRICE: np.int64, L_DISCOUNT: np.int64, L_TAX: np.int64, L_PARTKEY: np.int32,
    L_SUPPKEY: np.int32, L_SHIPMODE: np.uint8, L_SHIPINSTRUCT: np.uint8, P_BRAND: np.uint8,
    P_CONTAINER: np.uint8, P_SIZE: np.int32, S_NATIONKEY: np.uint8, F32_UNIFORM: np.float32,
    I32_UNIFORM: np.int32, I32_PERM: np.int32, I64_UNIFORM: np.int64, F64_UNIFORM: np.float64,
}

LINEITEM_COLS = {
    "l_shipdate": L_SHIPDATE, "l_returnflag": L_RETURNFLAG, "l_linestatus": L_LINESTATUS,
    "l_quantity": L_QUANTITY, "l_extendedprice": L_EXTENDEDPRICE, "l_discount": L_DISCOUNT,
    "l_tax": L_TAX, "l_partkey": L_PARTKEY, "l_suppkey": L_SUPPKEY, "l_shipmode": L_SHIPMODE,
    "l_shipinstruct": L_SHIPINSTRUCT,
}
PART_COLS = {"p_brand": P_BRAND, "p_container": P_CONTAINER, "p_size": P_SIZE}
SUPPLIER_COLS = {"s_nationkey": S_NATIONKEY}

# Order-preserving dictionaries [ext: TPC-H 4.2.2.13]; codes = sorted rank.
RETURNFLAG = ["A", "N", "R"]
LINESTATUS = ["F", "O"]
SHIPMODE = sorted(["REG AIR", "AIR", "RAIL", "SHIP", "TRUCK", "MAIL", "FOB"])
SHIPINSTRUCT = sorted(["DELIVER IN PERSON", "COLLECT COD", "NONE", "TAKE BACK RETURN"])
CONTAINER = sorted(f"{a} {b}" for a in ["SM", "LG", "MED", "JUMBO", "WRAP"]
                   for b in ["CASE", "BOX", "BAG", "JAR", "PKG", "PACK", "CAN", "DRUM"])
BRAND = [f"Brand#{m}{n}" for m in range(1, 6) for n in range(1, 6)]


def _lib():
    global _LIB
    if _LIB is None:
        path = os.path.join(_HERE, "libvdgen.so")
        if not os.path.exists(path):
            raise RuntimeError(f"{path} missing: run `make` (or __graft_entry__.build())")
        lib = ctypes.CDLL(path)
        lib.vdg_fill_host.restype = ctypes.c_int
        lib.vdg_fill_host.argtypes = [ctypes.c_int, ctypes.c_uint64, ctypes.c_double, ctypes.c_int64,
                                      ctypes.c_int64, ctypes.c_double, ctypes.c_int64, ctypes.c_int64,
                                      ctypes.c_void_p]
        lib.vdg_fill_device.restype = ctypes.c_int
        lib.vdg_fill_device.argtypes = [ctypes.c_int, ctypes.c_uint64, ctypes.c_double, ctypes.c_int64,
                                        ctypes.c_int64, ctypes.c_double, ctypes.c_int64, ctypes.c_int64,
                                        ctypes.c_void_p, ctypes.c_void_p]
        _LIB = lib
    return _LIB


def dtype_of(col: int):
    return _DTYPES[col]


def lineitem_rows(sf: float) -> int:
    return int(6000000.0 * sf + 0.5)


def part_rows(sf: float) -> int:
    return max(1, int(200000.0 * sf + 0.5))


def supplier_rows(sf: float) -> int:
    return max(1, int(10000.0 * sf + 0.5))


def host(col: int, n: int, row0: int = 0, *, sf: float = 1.0, seed: int = DEFAULT_SEED,
         p0: int = 0, p1: int = 0, fscale: float = 1.0, threads: int = 1) -> np.ndarray:
    """Rows [row0, row0+n) of column `col` as a numpy array (host generation).

    ``threads`` > 1 splits the row range over Python threads (the C loop
    releases the GIL); values do not depend on it (counter-based draws).
    """
    out = np.empty(int(n), dtype=_DTYPES[col])
    if n == 0:
        return out
    lib = _lib()
    if threads <= 1 or n < 1 << 20:
        rc = lib.vdg_fill_host(col, seed, sf, p0, p1, fscale, row0, n, out.ctypes.data)
        if rc != 0:
            raise ValueError(f"vdg_fill_host({col}) failed: {rc}")
        return out
    import concurrent.futures as cf
    step = (n + threads - 1) // threads
    item = out.itemsize

    def part(k):
        a = k * step
        b = min(n, a + step)
        if a >= b:
            return 0
        return lib.vdg_fill_host(col, seed, sf, p0, p1, fscale, row0 + a, b - a, out.ctypes.data + a * item)

    with cf.ThreadPoolExecutor(threads) as ex:
        for rc in ex.map(part, range(threads)):
            if rc != 0:
                raise ValueError(f"vdg_fill_host({col}) failed: {rc}")
    return out


def device(col: int, out_ptr: int, n: int, row0: int = 0, *, sf: float = 1.0, seed: int = DEFAULT_SEED,
           p0: int = 0, p1: int = 0, fscale: float = 1.0, stream: int = 0) -> None:
    """Fill `n` rows of column `col` into the device buffer at `out_ptr`."""
    rc = _lib().vdg_fill_device(col, seed, sf, p0, p1, fscale, row0, n, ctypes.c_void_p(out_ptr),
                                ctypes.c_void_p(stream))
    if rc != 0:
        raise RuntimeError(f"vdg_fill_device({col}) failed: {rc}")
