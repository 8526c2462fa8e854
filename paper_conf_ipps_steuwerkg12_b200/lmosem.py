"""Thin Python binding of the C ABI in ``include/lmosem.h`` (argument marshalling only).

Every step of the LM-OSEM subset iteration runs in ``liblmosem.so`` (sm_100a kernels +
NCCL); this module only converts torch tensors / numpy arrays to pointers. PyTorch
provides device memory, streams and the process group used to broadcast the NCCL id.
There is no CPU fallback: without the CUDA library or a GPU every call raises.
"""
from __future__ import annotations

import ctypes
import os

import numpy as np

_PKG = os.path.dirname(os.path.abspath(__file__))
# LMOSEM_LIB selects an in-tree A/B build of the same library (tools/ab_variants.py)
SO_PATH = os.environ.get("LMOSEM_LIB") or os.path.join(_PKG, "liblmosem.so")

OK, EINVAL, ENOMEM, ECUDA, ENCCL, ESTATE, EIO = range(7)
_NAMES = {0: "OK", 1: "EINVAL", 2: "ENOMEM", 3: "ECUDA", 4: "ENCCL", 5: "ESTATE", 6: "EIO"}
NCCL_ID_BYTES = 128

# every symbol include/lmosem.h declares (checked by tests/test_abi.py)
EXPORTS = (
    "lmosem_version", "lmosem_block_range", "lmosem_nccl_unique_id", "lmosem_init", "lmosem_set_stream",
    "lmosem_subset_step", "lmosem_reconstruct", "lmosem_reconstruct_host", "lmosem_error_image",
    "lmosem_forward", "lmosem_update", "lmosem_synchronize", "lmosem_set_timing", "lmosem_get_stats",
    "lmosem_destroy", "lmosem_last_error", "lmosem_set_slabs", "lmosem_get_slabs",
    "lmosem_sensitivity", "lmosem_set_norm", "lmosem_set_combine", "lmosem_get_combine",
    "lmosem_reconstruct_file", "lmosem_isd_block", "lmosem_loopback_create", "lmosem_loopback_destroy",
    "lmosem_init_loopback",
)
COMBINE_ALLREDUCE, COMBINE_ISD, COMBINE_FUSED = 1, 2, 3


class LmosemError(RuntimeError):
    def __init__(self, status: int, msg: str):
        super().__init__(f"lmosem {_NAMES.get(status, status)}: {msg}")
        self.status = status


class Dist(ctypes.Structure):
    _fields_ = [("rank", ctypes.c_int32), ("world", ctypes.c_int32), ("nccl_unique_id", ctypes.c_void_p)]


class Stats(ctypes.Structure):
    _fields_ = [("launches", ctypes.c_int64), ("subsets", ctypes.c_int64), ("events", ctypes.c_int64),
                ("timed_subsets", ctypes.c_int64), ("convert_ms", ctypes.c_double), ("project_ms", ctypes.c_double),
                ("combine_ms", ctypes.c_double), ("update_ms", ctypes.c_double), ("h2d_ms", ctypes.c_double),
                ("tune_fused_ms", ctypes.c_double), ("tune_isd_ms", ctypes.c_double),
                ("tune_allreduce_ms", ctypes.c_double)]

    def as_dict(self) -> dict:
        return {k: getattr(self, k) for k, _ in self._fields_}


_lib = None
_P = ctypes.c_void_p
_I64 = ctypes.c_int64
_I32 = ctypes.c_int32
_S = ctypes.c_int


def load(build_if_missing: bool = False) -> ctypes.CDLL:
    """Loads liblmosem.so (fails loudly if it is missing; no fallback)."""
    global _lib
    if _lib is not None:
        return _lib
    if build_if_missing:
        from . import build as _b
        _b.build()
    if not os.path.exists(SO_PATH):
        raise ImportError(f"{SO_PATH} not built: run `python -c 'import __graft_entry__ as g; g.build()'`")
    lib = ctypes.CDLL(SO_PATH)
    sig = {
        "lmosem_version": ([], ctypes.c_char_p),
        "lmosem_block_range": ([_I64, _I32, _I32, ctypes.POINTER(_I64), ctypes.POINTER(_I64)], _S),
        "lmosem_isd_block": ([_I64, _I32, _I32, ctypes.POINTER(_I64), ctypes.POINTER(_I64), ctypes.POINTER(_I64)], _S),
        "lmosem_nccl_unique_id": ([_P, ctypes.c_size_t], _S),
        "lmosem_init": ([ctypes.POINTER(_P), _P, _P, _P, ctypes.POINTER(Dist)], _S),
        "lmosem_loopback_create": ([_I32, ctypes.POINTER(_P)], _S),
        "lmosem_loopback_destroy": ([_P], _S),
        "lmosem_init_loopback": ([ctypes.POINTER(_P), _P, _P, _P, _P, _I32], _S),
        "lmosem_set_stream": ([_P, _P], _S),
        "lmosem_set_slabs": ([_P, _I32], _S),
        "lmosem_set_combine": ([_P, _I32], _S),
        "lmosem_get_combine": ([_P], _I32),
        "lmosem_get_slabs": ([_P], _I32),
        "lmosem_subset_step": ([_P, _P, _I64, _P], _S),
        "lmosem_reconstruct": ([_P, _P, _P, _I32, _I32, _P], _S),
        "lmosem_reconstruct_host": ([_P, _P, _P, _I32, _I32, _P], _S),
        "lmosem_reconstruct_file": ([_P, ctypes.c_char_p, _P, _I32, _I32, _P], _S),
        "lmosem_error_image": ([_P, _P, _I64, _P, _P], _S),
        "lmosem_forward": ([_P, _P, _I64, _P, _P], _S),
        "lmosem_update": ([_P, _P, _P], _S),
        "lmosem_sensitivity": ([_P, _P, _I64, _P], _S),
        "lmosem_set_norm": ([_P, _P], _S),
        "lmosem_synchronize": ([_P], _S),
        "lmosem_set_timing": ([_P, _I32], _S),
        "lmosem_get_stats": ([_P, ctypes.POINTER(Stats)], _S),
        "lmosem_destroy": ([_P], _S),
        "lmosem_last_error": ([_P], ctypes.c_char_p),
    }
    for name, (args, res) in sig.items():
        fn = getattr(lib, name)
        fn.argtypes = args
        fn.restype = res
    _lib = lib
    return lib


def version() -> str:
    return load().lmosem_version().decode()


def block_range(n: int, rank: int, world: int) -> tuple[int, int]:
    """Block distribution of n events over world ranks."""
    b, e = _I64(), _I64()
    st = load().lmosem_block_range(int(n), int(rank), int(world), ctypes.byref(b), ctypes.byref(e))
    if st != OK:
        raise LmosemError(st, "block_range: bad arguments")
    return b.value, e.value


def isd_block(n_bricks: int, rank: int, world: int) -> tuple[int, int, int]:
    """(begin, end, alloc) of rank's ISD brick block."""
    b, e, a = _I64(), _I64(), _I64()
    st = load().lmosem_isd_block(int(n_bricks), int(rank), int(world), ctypes.byref(b), ctypes.byref(e),
                                 ctypes.byref(a))
    if st != OK:
        raise LmosemError(st, "isd_block: bad arguments")
    return b.value, e.value, a.value


def nccl_unique_id() -> bytes:
    buf = ctypes.create_string_buffer(NCCL_ID_BYTES)
    st = load().lmosem_nccl_unique_id(buf, NCCL_ID_BYTES)
    if st != OK:
        raise LmosemError(st, "ncclGetUniqueId failed")
    return buf.raw


def _dev_ptr(t, dtype_name: str, numel: int | None = None) -> int:
    import torch
    if not isinstance(t, torch.Tensor) or not t.is_cuda:
        raise TypeError("expected a CUDA torch.Tensor")
    if str(t.dtype) != f"torch.{dtype_name}":
        raise TypeError(f"expected {dtype_name}, got {t.dtype}")
    if not t.is_contiguous():
        raise ValueError("tensor must be contiguous")
    if numel is not None and t.numel() != numel:
        raise ValueError(f"expected {numel} elements, got {t.numel()}")
    return t.data_ptr()


def _host_ptr(a, numel: int | None = None) -> int:
    import torch
    if isinstance(a, torch.Tensor):
        if a.is_cuda or a.dtype != torch.float32 or not a.is_contiguous():
            raise TypeError("expected a contiguous float32 CPU tensor")
        if numel is not None and a.numel() != numel:
            raise ValueError(f"expected {numel} elements")
        return a.data_ptr()
    if not (isinstance(a, np.ndarray) and a.dtype == np.float32 and a.flags.c_contiguous):
        raise TypeError("expected a contiguous float32 numpy array")
    if numel is not None and a.size != numel:
        raise ValueError(f"expected {numel} elements")
    return a.ctypes.data


class Loopback:
    """An emulated world of `world` ranks on one GPU (include/lmosem.h, "Emulated world"):
    pass ``loopback=(group, rank)`` to Reconstructor, one context per rank, and drive each
    rank's collective calls from its own thread. Test transport: the contexts run the same
    combine code as NCCL ranks. Close the contexts before the group."""

    def __init__(self, world: int):
        self._lib = load()
        h = _P()
        st = self._lib.lmosem_loopback_create(int(world), ctypes.byref(h))
        if st != OK:
            raise LmosemError(st, f"loopback_create({world})")
        self._h = h
        self.world = int(world)

    def close(self):
        if getattr(self, "_h", None) is not None and self._h.value:
            st = self._lib.lmosem_loopback_destroy(self._h)
            if st != OK:
                raise LmosemError(st, "loopback_destroy: contexts still registered")
            self._h = _P()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


class Reconstructor:
    """One LM-OSEM context (one GPU / rank). See include/lmosem.h for semantics.

    ``norm``: V float32 sensitivity image (CUDA tensor or host array), copied at init.
    ``dist``: None for one GPU, or (rank, world, nccl_id_bytes) for a collective context.
    ``stream``: torch.cuda.Stream to enqueue on (default: torch's current stream).
    ``loopback``: (Loopback, rank) for a rank of an emulated world on this GPU (tests).
    """

    def __init__(self, dims, voxel_mm, norm, dist=None, stream=None, loopback=None):
        import torch
        lib = load()
        if not torch.cuda.is_available():
            raise RuntimeError("lmosem needs a CUDA device (no CPU fallback)")
        self._lib = lib
        self.dims = tuple(int(d) for d in dims)
        self.voxel_mm = tuple(float(v) for v in voxel_mm)
        self.V = self.dims[0] * self.dims[1] * self.dims[2]
        d = (ctypes.c_int32 * 3)(*self.dims)
        v = (ctypes.c_double * 3)(*self.voxel_mm)
        if isinstance(norm, torch.Tensor) and norm.is_cuda:
            nptr = _dev_ptr(norm, "float32", self.V)
            torch.cuda.current_stream().synchronize()
        else:
            nptr = _host_ptr(norm, self.V)
        self._keep = None
        dptr = None
        if dist is not None:
            rank, world, uid = dist
            self._keep = ctypes.create_string_buffer(bytes(uid), NCCL_ID_BYTES)
            dptr = ctypes.byref(Dist(int(rank), int(world), ctypes.cast(self._keep, ctypes.c_void_p)))
        h = _P()
        if dist is not None and loopback is not None:
            raise ValueError("dist and loopback are exclusive")
        if loopback is not None:
            group, rank = loopback
            self._group = group  # the group outlives this context
            st = lib.lmosem_init_loopback(ctypes.byref(h), d, v, nptr, group._h, int(rank))
        else:
            st = lib.lmosem_init(ctypes.byref(h), d, v, nptr, dptr)
        if st != OK:
            raise LmosemError(st, lib.lmosem_last_error(None).decode())
        self._h = h
        if loopback is not None:
            self.rank, self.world = int(loopback[1]), loopback[0].world
        else:
            self.rank, self.world = (0, 1) if dist is None else (int(dist[0]), int(dist[1]))
        self.set_stream(stream if stream is not None else torch.cuda.current_stream())

    # -- plumbing
    def _check(self, st: int):
        if st != OK:
            raise LmosemError(st, self._lib.lmosem_last_error(self._h).decode())

    def set_stream(self, stream):
        self._stream = stream
        # torch's default stream has handle 0 = the CUDA default stream for the library
        self._check(self._lib.lmosem_set_stream(self._h, _P(stream.cuda_stream)))

    def close(self):
        if getattr(self, "_h", None) is not None and self._h.value:
            self._lib.lmosem_destroy(self._h)
            self._h = _P()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.close()

    # -- the path (device buffers; stream-ordered)
    @staticmethod
    def _events_ptr(events) -> tuple[int, int]:
        n = events.numel() // 6 if events.numel() else 0
        if events.numel() != 6 * n:
            raise ValueError("events must hold 6 floats per event")
        return (_dev_ptr(events, "float32") if n else 0), n

    def subset_step(self, events, f):
        """One subset iteration: step 1 (this rank's block), c all-reduce, step 2 on f."""
        ep, n = self._events_ptr(events)
        self._check(self._lib.lmosem_subset_step(self._h, ep, n, _dev_ptr(f, "float32", self.V)))

    @staticmethod
    def _offsets(offsets, n: int) -> np.ndarray:
        """Subset offsets as int64; the C side cannot see the event count, so the binding
        checks that every subset lies inside the n events it was given."""
        off = np.ascontiguousarray(offsets, dtype=np.int64)
        if off.ndim != 1 or off.size < 1:
            raise ValueError("offsets must be a 1-D array of n_subsets + 1 entries")
        if off[0] < 0 or off[-1] > n or np.any(np.diff(off) < 0):
            raise ValueError(f"offsets must be non-decreasing within [0, {n}]")
        return off

    def reconstruct(self, events, offsets, n_iterations, f):
        """n_iterations passes over subsets events[offsets[l]:offsets[l+1]] (in events)."""
        ep, n = self._events_ptr(events)
        off = self._offsets(offsets, n)
        self._check(self._lib.lmosem_reconstruct(self._h, ep, off.ctypes.data, off.size - 1, int(n_iterations),
                                                 _dev_ptr(f, "float32", self.V)))

    def resume(self, events, offsets, n_iterations, f, start_iteration: int, start_subset: int):
        """Checkpoint / resume: continue a reconstruction of n_iterations passes
        from a checkpoint taken after subset start_subset - 1 of iteration start_iteration
        (f = the checkpointed image, e.g. copied out after a reconstruct call that stopped
        there): the rest of that iteration, then the remaining full iterations — the same
        sequence of subset iterations as one uninterrupted lmosem_reconstruct call (two calls
        of the C ABI; nothing is computed here)."""
        off = self._offsets(offsets, self._events_ptr(events)[1])
        L = off.size - 1
        if not (0 <= start_iteration <= n_iterations and 0 <= start_subset <= L):
            raise ValueError("start outside the reconstruction")
        if start_iteration < n_iterations and start_subset < L:
            self.reconstruct(events, off[start_subset:], 1, f)
            start_iteration += 1
        if start_iteration < n_iterations:
            self.reconstruct(events, off, n_iterations - start_iteration, f)

    def reconstruct_host(self, events, offsets, n_iterations, f):
        """Host events + host f (in/out); H2D streaming overlapped with projection."""
        n = (events.numel() if hasattr(events, "numel") else np.asarray(events).size) // 6
        off = self._offsets(offsets, n)
        self._check(self._lib.lmosem_reconstruct_host(self._h, _host_ptr(events), off.ctypes.data, off.size - 1,
                                                      int(n_iterations), _host_ptr(f, self.V)))

    def reconstruct_file(self, path, offsets, n_iterations, f):
        """Events streamed from a raw lmosem_event file (24 B records), f a CUDA tensor."""
        off = np.ascontiguousarray(offsets, dtype=np.int64)
        self._check(self._lib.lmosem_reconstruct_file(self._h, os.fsencode(path), off.ctypes.data, off.size - 1,
                                                      int(n_iterations), _dev_ptr(f, "float32", self.V)))

    def error_image(self, events, f, c_out):
        ep, n = self._events_ptr(events)
        self._check(self._lib.lmosem_error_image(self._h, ep, n, _dev_ptr(f, "float32", self.V),
                                                 _dev_ptr(c_out, "float32", self.V)))

    def forward(self, events, f, fp_out):
        ep, n = self._events_ptr(events)
        self._check(self._lib.lmosem_forward(self._h, ep, n, _dev_ptr(f, "float32", self.V),
                                             _dev_ptr(fp_out, "float32", n) if n else 0))

    def sensitivity(self, events, s_out):
        """s_out_j = sum_i a_ij over the given LORs (back-projection of ones)."""
        ep, n = self._events_ptr(events)
        self._check(self._lib.lmosem_sensitivity(self._h, ep, n, _dev_ptr(s_out, "float32", self.V)))

    def set_norm(self, norm):
        """Replaces the norm image (CUDA tensor or host float32 array, V elements)."""
        import torch
        if isinstance(norm, torch.Tensor) and norm.is_cuda:
            ptr = _dev_ptr(norm, "float32", self.V)
        else:
            ptr = _host_ptr(norm, self.V)
        self._check(self._lib.lmosem_set_norm(self._h, ptr))

    def update(self, f, c):
        self._check(self._lib.lmosem_update(self._h, _dev_ptr(f, "float32", self.V), _dev_ptr(c, "float32", self.V)))

    def set_combine(self, mode: int):
        """0 = auto, COMBINE_ALLREDUCE, COMBINE_ISD or COMBINE_FUSED (collective; see lmosem.h)."""
        self._check(self._lib.lmosem_set_combine(self._h, int(mode)))

    @property
    def combine(self) -> int:
        return int(self._lib.lmosem_get_combine(self._h))

    def set_slabs(self, n_slabs: int):
        """z-slab passes for step 1 (0 = automatic from the L2 budget); see lmosem.h."""
        self._check(self._lib.lmosem_set_slabs(self._h, int(n_slabs)))

    @property
    def slabs(self) -> int:
        return int(self._lib.lmosem_get_slabs(self._h))

    def synchronize(self):
        self._check(self._lib.lmosem_synchronize(self._h))

    def set_timing(self, enable: bool):
        self._check(self._lib.lmosem_set_timing(self._h, 1 if enable else 0))

    def stats(self) -> dict:
        s = Stats()
        self._check(self._lib.lmosem_get_stats(self._h, ctypes.byref(s)))
        return s.as_dict()


def make_dist(rank: int, world: int, group=None) -> tuple[int, int, bytes] | None:
    """NCCL id from rank 0, broadcast with torch.distributed (any backend). None for world 1."""
    if world <= 1:
        return None
    import torch.distributed as dist
    obj = [nccl_unique_id() if rank == 0 else None]
    dist.broadcast_object_list(obj, src=0, group=group)
    return (rank, world, obj[0])
