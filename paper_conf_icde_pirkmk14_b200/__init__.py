"""B200-native Approximate & Refine (A&R) over bitwise-distributed (BWD) columns.

The hot path of H. Pirk, S. Manegold, M. Kersten, "Waste Not... Efficient
Co-Processing of Relational Data" (ICDE 2014): BWD decomposition (a1),
approximate selection with relaxed bounds + stable compaction (a2, a3),
row-sharded count exchange (a4), positional refine (a5) and exact SUM (a6),
as hand-written sm_100a CUDA behind the C ABI in include/ar.h.

`_ar` is the ctypes binding (same names as the C entry points); `column`
holds the torch memory / stream plumbing; `dist` the torch.distributed glue
for the NCCL communicator.
"""
from . import _ar  # noqa: F401
from ._ar import ARError, load  # noqa: F401

__all__ = ["_ar", "ARError", "load"]
