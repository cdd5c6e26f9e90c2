"""voodoo-b200: the data-parallel hot path of Voodoo's compiled vector algebra
(Pirk, Moll, Zaharia, Madden, PVLDB 9(14) 2016) as hand-written sm_100a CUDA
behind the C ABI of include/vd.h.

* :mod:`.vd`    -- ctypes binding of libvd.so (marshalling only)
* :mod:`.plans` -- vd_pipeline descriptors of the TPC-H-shaped workloads
* :mod:`.dist`  -- one process per GPU: row-range sharding + partial merge
"""
from . import vd  # noqa: F401  (raises ImportError if libvd.so is missing)

__all__ = ["vd"]
