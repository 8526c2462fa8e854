"""Plain float64 CPU LM-OSEM oracle (ctypes wrapper over ``oracle.c``).

TEST INFRASTRUCTURE ONLY: only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this package. The product path
(``paper_conf_ipps_steuwerkg12_b200``) never imports it and shares no code with it.

Follows PAPER.md §IV Listing 2 (lines 452-470) with the readings S1-S17 of DESIGN.md;
see ``oracle.h`` for the per-function citations. Parity pins live in
``tests/test_oracle_pins.py``.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liboracle.so")


def build(force: bool = False) -> str:
    """Compile liboracle.so (gcc -O2 -fopenmp; strict IEEE float64, no fast-math)."""
    src = os.path.join(_HERE, "oracle.c")
    hdr = os.path.join(_HERE, "oracle.h")
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < max(os.path.getmtime(src), os.path.getmtime(hdr)):
        tmp = _SO + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O2", "-fno-fast-math", "-ffp-contract=off", "-fopenmp", "-fPIC",
                               "-shared", "-std=c11", "-o", tmp, src, "-lm"])
        os.replace(tmp, _SO)
    return _SO


class Geom(ctypes.Structure):
    _fields_ = [("nx", ctypes.c_int32), ("ny", ctypes.c_int32), ("nz", ctypes.c_int32),
                ("vx", ctypes.c_double), ("vy", ctypes.c_double), ("vz", ctypes.c_double)]


def geom(dims, voxel_mm) -> Geom:
    return Geom(int(dims[0]), int(dims[1]), int(dims[2]),
                float(voxel_mm[0]), float(voxel_mm[1]), float(voxel_mm[2]))


_lib = None
_P = ctypes.c_void_p


def _load():
    global _lib
    if _lib is None:
        # LMOSEM_ORACLE_SO: a prebuilt variant of this library (tests/test_oracle_mutants.py
        # loads deliberately broken copies to check that the pins catch them)
        lib = ctypes.CDLL(os.environ.get("LMOSEM_ORACLE_SO") or build())
        G = ctypes.POINTER(Geom)
        for name in ("oracle_siddon_path", "oracle_boxclip_path"):
            fn = getattr(lib, name)
            fn.argtypes = [G, _P, _P, _P, _P, ctypes.c_int64]
            fn.restype = ctypes.c_int64
        lib.oracle_forward.argtypes = [G, _P, ctypes.c_int64, _P, _P]
        lib.oracle_error_image.argtypes = [G, _P, ctypes.c_int64, _P, _P]
        lib.oracle_update.argtypes = [ctypes.c_int64, _P, _P, _P]
        lib.oracle_sensitivity.argtypes = [G, _P, ctypes.c_int64, _P]
        lib.oracle_subset_step.argtypes = [G, _P, ctypes.c_int64, _P, _P]
        lib.oracle_subset_step.restype = ctypes.c_int
        lib.oracle_reconstruct.argtypes = [G, _P, _P, ctypes.c_int32, ctypes.c_int32, _P, _P]
        lib.oracle_reconstruct.restype = ctypes.c_int
        lib.oracle_set_threads.argtypes = [ctypes.c_int32]
        lib.oracle_get_threads.restype = ctypes.c_int32
        _lib = lib
    return _lib


def _f32(a) -> np.ndarray:
    return np.ascontiguousarray(a, dtype=np.float32)


def _f64(a) -> np.ndarray:
    return np.ascontiguousarray(a, dtype=np.float64)


def _path(fn, g: Geom, p1, p2):
    p1 = _f64(p1)
    p2 = _f64(p2)
    cap = int(g.nx) * g.ny * g.nz + 8 if fn == "oracle_boxclip_path" else g.nx + g.ny + g.nz + 8
    coord = np.empty(cap, np.int32)
    ln = np.empty(cap, np.float64)
    m = getattr(_load(), fn)(ctypes.byref(g), p1.ctypes.data, p2.ctypes.data, coord.ctypes.data, ln.ctypes.data, cap)
    if m < 0:
        raise RuntimeError(f"{fn}: capacity exceeded")
    return coord[:m].copy(), ln[:m].copy()


def siddon_path(g: Geom, p1, p2):
    """compute_path (Listing 2 line 7): (coord int32[m], len float64[m]) in traversal order."""
    return _path("oracle_siddon_path", g, p1, p2)


def boxclip_path(g: Geom, p1, p2):
    """Brute-force per-voxel box clip (tiny volumes only): (coord, len) in increasing coord."""
    return _path("oracle_boxclip_path", g, p1, p2)


def forward(g: Geom, events, f) -> np.ndarray:
    """fp_i = sum_j a_ij f_j (Listing 2 lines 9-10), float64[n]."""
    ev = _f32(events).reshape(-1, 6)
    f = _f64(f)
    fp = np.empty(ev.shape[0], np.float64)
    _load().oracle_forward(ctypes.byref(g), ev.ctypes.data, ev.shape[0], f.ctypes.data, fp.ctypes.data)
    return fp


def error_image(g: Geom, events, f) -> np.ndarray:
    """Step 1 (Listing 2 lines 5-13) from c = 0: float64[V]."""
    ev = _f32(events).reshape(-1, 6)
    f = _f64(f)
    c = np.empty(int(g.nx) * g.ny * g.nz, np.float64)
    _load().oracle_error_image(ctypes.byref(g), ev.ctypes.data, ev.shape[0], f.ctypes.data, c.ctypes.data)
    return c


def sensitivity(g: Geom, events) -> np.ndarray:
    """s_j = sum_i a_ij over the given LORs (back-projection of ones), float64[V]."""
    ev = _f32(events).reshape(-1, 6)
    out = np.empty(int(g.nx) * g.ny * g.nz, np.float64)
    _load().oracle_sensitivity(ctypes.byref(g), ev.ctypes.data, ev.shape[0], out.ctypes.data)
    return out


def update(f, c, s) -> np.ndarray:
    """Step 2 (Listing 2 lines 16-17 with norm): returns the new float64 f."""
    f = _f64(f).copy()
    c = _f64(c)
    s = _f32(s)
    _load().oracle_update(f.size, f.ctypes.data, c.ctypes.data, s.ctypes.data)
    return f


def subset_step(g: Geom, events, s, f) -> np.ndarray:
    """One subset iteration; returns the new float64 f (input untouched)."""
    ev = _f32(events).reshape(-1, 6)
    f = _f64(f).copy()
    s = _f32(s)
    if _load().oracle_subset_step(ctypes.byref(g), ev.ctypes.data, ev.shape[0], s.ctypes.data, f.ctypes.data):
        raise MemoryError("oracle_subset_step")
    return f


def reconstruct(g: Geom, events, offsets, n_iterations, s, f0) -> np.ndarray:
    """I iterations over the subsets events[offsets[l]:offsets[l+1]]; returns float64 f."""
    ev = _f32(events).reshape(-1, 6)
    off = np.ascontiguousarray(offsets, dtype=np.int64)
    f = _f64(f0).copy()
    s = _f32(s)
    rc = _load().oracle_reconstruct(ctypes.byref(g), ev.ctypes.data, off.ctypes.data, off.size - 1,
                                    int(n_iterations), s.ctypes.data, f.ctypes.data)
    if rc:
        raise MemoryError("oracle_reconstruct")
    return f


def set_threads(n: int) -> None:
    _load().oracle_set_threads(int(n))


def get_threads() -> int:
    return int(_load().oracle_get_threads())
