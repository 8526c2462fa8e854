#!/usr/bin/env python
"""Offline layout analysis: unique 32-byte sectors per 32-piece instruction,
path order, for C2 paths under candidate image layouts. Uses the oracle's paths (analysis
tooling, not product code). Lives under tests/ because it runs the oracle (test infrastructure). Usage: python tests/analysis/sector_sim.py [n_events] [config]"""
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import lmgen  # noqa: E402
import oracle  # noqa: E402


def sector_keys(ix, iy, iz, dom, layout):
    if layout == "brick 2x2x2":
        return (ix >> 1) + 1000 * ((iy >> 1) + 1000 * (iz >> 1))
    if layout == "x-major rows of 8":
        return (ix >> 3) + 1000 * (iy + 1000 * iz)
    if layout[0] == "abs":  # one layout for every LOR: brick extents along (x, y, z)
        _, ex, ey, ez = layout
        return (ix // ex) + 1000 * ((iy // ey) + 1000 * (iz // ez))
    ea, eb, ec = layout  # per-dominant-axis layouts: extents along (a, b, c)
    ax = [ix, iy, iz]
    b = 1 if dom == 0 else 0
    c = 1 if dom == 2 else 2
    return (ax[dom] // ea) + 1000 * ((ax[b] // eb) + 1000 * (ax[c] // ec))


def main():
    n = int(sys.argv[1]) if len(sys.argv) > 1 else 3000
    cfg = lmgen.CONFIGS[sys.argv[2] if len(sys.argv) > 2 else "C2"]
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    nx, ny, _ = cfg.dims
    ev = lmgen.subset_events(cfg, 0, n)
    layouts = ["brick 2x2x2", "x-major rows of 8", (8, 1, 1), (4, 1, 2), (4, 2, 1),
               ("abs", 4, 2, 1), ("abs", 2, 4, 1), ("abs", 4, 1, 2), ("abs", 1, 4, 2), ("abs", 2, 1, 4),
               ("abs", 1, 2, 4), ("abs", 8, 1, 1), ("abs", 1, 1, 8)]
    sectors = {str(L): 0 for L in layouts}
    pieces = 0
    for e in ev:
        co, _ = oracle.siddon_path(g, e[:3].astype(float), e[3:].astype(float))
        if len(co) == 0:
            continue
        ix, iy, iz = co % nx, (co // nx) % ny, co // (nx * ny)
        dom = int(np.argmax(np.abs(e[3:] - e[:3]) / np.asarray(cfg.voxel_mm)))
        pieces += len(co)
        for L in layouts:
            k = sector_keys(ix, iy, iz, dom, L)
            sectors[str(L)] += sum(len(np.unique(k[s:s + 32])) for s in range(0, len(k), 32))
    for L in layouts:
        print(f"{str(L):20s} pieces per sector {pieces / sectors[str(L)]:.3f}")


if __name__ == "__main__":
    main()
