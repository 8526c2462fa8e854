"""Seeded synthetic list-mode PET inputs (events + norm image) for LM-OSEM.

Input generator shared by the CPU oracle (``oracle/``) and the CUDA path. It holds
none of the LM-OSEM arithmetic: it only draws emission points, directions and the
scanner-geometry acceptance that defines the norm image (see ``lmgen.h``).

Configs C1..C5 are BASELINE.json ``configs[0..4]`` with the recipe of SURVEY.md §8(d)
and DESIGN.md "Input recipe". The workload shape is PAPER.md §IV.C (lines 586-591):
150x150x280 voxels, ~10^6 events per subset, ~10^2 subsets.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from dataclasses import dataclass, field

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liblmgen.so")
_MAX_SPHERES = 8


def build(force: bool = False) -> str:
    """Compile liblmgen.so with gcc (-O2, OpenMP, no fast-math so bytes are reproducible)."""
    src = os.path.join(_HERE, "lmgen.c")
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < max(
        os.path.getmtime(src), os.path.getmtime(os.path.join(_HERE, "lmgen.h"))
    ):
        tmp = _SO + f".tmp{os.getpid()}"
        subprocess.check_call(
            ["gcc", "-O2", "-fno-fast-math", "-ffp-contract=off", "-fopenmp", "-fPIC", "-shared",
             "-std=c11", "-D_GNU_SOURCE", "-o", tmp, src, "-lm"]
        )
        os.replace(tmp, _SO)
    return _SO


class _Cfg(ctypes.Structure):
    _fields_ = [
        ("nx", ctypes.c_int32), ("ny", ctypes.c_int32), ("nz", ctypes.c_int32),
        ("vx", ctypes.c_double), ("vy", ctypes.c_double), ("vz", ctypes.c_double),
        ("h", ctypes.c_double), ("hz", ctypes.c_double),
        ("bg_kind", ctypes.c_int32),
        ("bg_r", ctypes.c_double), ("bg_half_len", ctypes.c_double), ("bg_act", ctypes.c_double),
        ("n_spheres", ctypes.c_int32),
        ("spheres", (ctypes.c_double * 5) * _MAX_SPHERES),
        ("hot_frac", ctypes.c_double), ("hot_r", ctypes.c_double),
        ("dir_mode", ctypes.c_int32),
        ("cos_lo", ctypes.c_double), ("cos_hi", ctypes.c_double), ("az_jitter_deg", ctypes.c_double),
        ("seed", ctypes.c_uint64),
        ("norm_dirs", ctypes.c_int32),
    ]


@dataclass(frozen=True)
class Config:
    """One synthetic workload. ``dims`` = (nx, ny, nz), ``voxel_mm`` = (vx, vy, vz)."""

    name: str
    dims: tuple
    voxel_mm: tuple
    h: float
    hz: float
    n_events: int          # events per subset (N)
    n_subsets: int         # L
    n_iterations: int      # I
    seed: int
    bg_kind: int = 0       # 0 cylinder, 1 sphere
    bg_r: float = 60.0
    bg_half_len: float = 130.0
    bg_act: float = 1.0
    spheres: tuple = ()    # ((cx, cy, cz, r, act), ...)
    hot_frac: float = 0.0
    hot_r: float = 0.0
    dir_mode: int = 0
    cos_lo: float = 0.0
    cos_hi: float = 0.0
    az_jitter_deg: float = 0.0
    norm_dirs: int = 257
    note: str = field(default="", compare=False)

    @property
    def n_voxels(self) -> int:
        return int(self.dims[0]) * int(self.dims[1]) * int(self.dims[2])

    def _c(self) -> _Cfg:
        c = _Cfg()
        c.nx, c.ny, c.nz = (int(d) for d in self.dims)
        c.vx, c.vy, c.vz = (float(v) for v in self.voxel_mm)
        c.h, c.hz = float(self.h), float(self.hz)
        c.bg_kind, c.bg_r, c.bg_half_len, c.bg_act = self.bg_kind, self.bg_r, self.bg_half_len, self.bg_act
        if len(self.spheres) > _MAX_SPHERES:
            raise ValueError("too many spheres")
        c.n_spheres = len(self.spheres)
        for i, s in enumerate(self.spheres):
            for k in range(5):
                c.spheres[i][k] = float(s[k])
        c.hot_frac, c.hot_r = self.hot_frac, self.hot_r
        c.dir_mode, c.cos_lo, c.cos_hi, c.az_jitter_deg = self.dir_mode, self.cos_lo, self.cos_hi, self.az_jitter_deg
        c.seed = int(self.seed)
        c.norm_dirs = int(self.norm_dirs)
        return c


_C2_SPHERES = (
    (20.0, 0.0, -60.0, 5.0, 4.0),
    (-25.0, 15.0, 0.0, 8.0, 4.0),
    (0.0, -30.0, 60.0, 12.0, 4.0),
    (0.0, 25.0, 40.0, 10.0, 0.0),   # cold insert
)

CONFIGS = {
    # BASELINE.json configs[0]: tiny, oracle finishes in seconds
    "C1": Config("C1", (16, 16, 16), (1.0, 1.0, 1.0), h=12.0, hz=8.0, n_events=10_000, n_subsets=2,
                 n_iterations=1, seed=1, bg_kind=1, bg_r=6.0, spheres=((2.0, -1.0, 1.0, 2.0, 4.0),),
                 norm_dirs=2049, note="tiny"),
    # configs[1]: paper-shaped, 1 GPU — the bench workload
    "C2": Config("C2", (150, 150, 280), (1.0, 1.0, 1.0), h=100.0, hz=140.0, n_events=1_000_000,
                 n_subsets=10, n_iterations=1, seed=2, spheres=_C2_SPHERES, note="paper-shaped"),
    # configs[2]: = C2, block-distributed on 2/4/8 GPUs
    "C3": Config("C3", (150, 150, 280), (1.0, 1.0, 1.0), h=100.0, hz=140.0, n_events=1_000_000,
                 n_subsets=10, n_iterations=1, seed=2, spheres=_C2_SPHERES, note="paper-shaped, P>1"),
    # configs[3]: 300x300x560 at 0.5 mm (c, f exceed L2), 10^7 events per subset
    "C4": Config("C4", (300, 300, 560), (0.5, 0.5, 0.5), h=100.0, hz=140.0, n_events=10_000_000,
                 n_subsets=10, n_iterations=1, seed=3, spheres=_C2_SPHERES, norm_dirs=129, note="scaled"),
    # configs[4]: skewed geometry — long oblique LORs, hot-spot contention
    "C5": Config("C5", (150, 150, 280), (1.0, 1.0, 1.0), h=100.0, hz=600.0, n_events=1_000_000,
                 n_subsets=10, n_iterations=1, seed=4, spheres=_C2_SPHERES, hot_frac=0.5, hot_r=3.0,
                 dir_mode=1, cos_lo=0.5, cos_hi=0.85, az_jitter_deg=10.0, note="skewed"),
}

_lib = None


def _load():
    global _lib
    if _lib is None:
        _lib = ctypes.CDLL(build())
        _lib.lmgen_events.argtypes = [ctypes.POINTER(_Cfg), ctypes.c_int64, ctypes.c_int64, ctypes.c_void_p]
        _lib.lmgen_events.restype = ctypes.c_int
        _lib.lmgen_norm.argtypes = [ctypes.POINTER(_Cfg), ctypes.c_void_p]
        _lib.lmgen_norm.restype = ctypes.c_int
    return _lib


def events(cfg: Config, first: int, count: int, out: np.ndarray | None = None) -> np.ndarray:
    """Events [first, first+count) as a (count, 6) float32 array (x1,y1,z1,x2,y2,z2 in mm)."""
    if out is None:
        out = np.empty((count, 6), dtype=np.float32)
    assert out.dtype == np.float32 and out.flags.c_contiguous and out.size >= 6 * count
    c = cfg._c()
    rc = _load().lmgen_events(ctypes.byref(c), int(first), int(count), out.ctypes.data)
    if rc != 0:
        raise RuntimeError(f"lmgen_events failed ({rc})")
    return out


def subset_events(cfg: Config, subset: int, count: int | None = None) -> np.ndarray:
    """Events of subset l: a contiguous block of the event list."""
    n = cfg.n_events if count is None else count
    return events(cfg, subset * cfg.n_events, n)


def norm(cfg: Config) -> np.ndarray:
    """The sensitivity (norm) image s, V float32, x fastest."""
    out = np.empty(cfg.n_voxels, dtype=np.float32)
    c = cfg._c()
    if _load().lmgen_norm(ctypes.byref(c), out.ctypes.data) != 0:
        raise RuntimeError("lmgen_norm failed")
    return out


def with_(cfg: Config, **kw) -> Config:
    """A copy of ``cfg`` with fields replaced (e.g. a smaller ``n_events`` for a sample)."""
    d = {k: getattr(cfg, k) for k in cfg.__dataclass_fields__}
    d.update(kw)
    return Config(**d)
