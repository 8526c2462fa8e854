"""B200-native LM-OSEM subset iteration (Steuwer, Kegel, Gorlatch, IPDPSW 2012, §IV).

The hot path — Siddon traversal, forward projection, atomic back-projection, the
cross-GPU combine of the error image and the image update — runs in ``liblmosem.so``
(hand-written sm_100a CUDA + NCCL) behind the C ABI of ``include/lmosem.h``;
``lmosem`` is the thin ctypes binding. There is no CPU fallback.
"""
from .lmosem import (EXPORTS, LmosemError, Loopback, Reconstructor, block_range, isd_block, load, make_dist,  # noqa: F401
                     nccl_unique_id, version)

__all__ = ["Reconstructor", "Loopback", "LmosemError", "block_range", "isd_block", "load", "make_dist", "nccl_unique_id",
           "version"]
