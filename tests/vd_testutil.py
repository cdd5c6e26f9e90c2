"""Shared helpers for the test suite (golden fixtures, input recipes)."""
import json
import os

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
GOLDEN = os.path.join(ROOT, "tests", "golden")


def load_golden(name):
    with open(os.path.join(GOLDEN, name)) as f:
        return json.load(f)


# ---- GPU-test helpers (imported only by -m gpu tests) -------------------------
def cuda_tensor(a):
    import numpy as np
    import torch
    return torch.from_numpy(np.ascontiguousarray(a)).cuda()


def minmax(a):
    import numpy as np
    a = np.asarray(a)
    return (int(a.min()), int(a.max())) if a.size else (0, 0)


EPS_BY_DTYPE = {"uint8": 0xFF, "int32": -(2**31), "int64": -(2**63)}


def with_eps(a, frac, seed):
    """Copy of `a` with a fraction of slots set to the dtype's epsilon sentinel."""
    import numpy as np
    a = np.array(a, copy=True)
    rng = np.random.default_rng(seed)
    m = rng.random(a.size) < frac
    if a.dtype.kind == "f":
        a[m] = np.nan
    else:
        a[m] = EPS_BY_DTYPE[a.dtype.name]
    return a, m


def i128_from_bytes(b, k):
    import struct
    lo, hi = struct.unpack_from("<Qq", b, 16 * k)
    return hi * (1 << 64) + lo
