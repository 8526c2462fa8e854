#!/usr/bin/env python
"""Device timeline of one lmosem_reconstruct_host call at C2 (CUPTI through torch.profiler:
the library's kernels and copies): where the wall time beyond the device-resident
reconstruction goes (diagnostic)."""
import json
import sys
import time

import numpy as np
import torch
from torch.profiler import ProfilerActivity, profile

import lmgen
import paper_conf_ipps_steuwerkg12_b200 as pkg


def main():
    cfg = lmgen.CONFIGS["C2"]
    ev = lmgen.events(cfg, 0, cfg.n_events * cfg.n_subsets)
    s = lmgen.norm(cfg)
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, torch.from_numpy(s).cuda())
    evh = torch.from_numpy(ev).pin_memory()
    fh = torch.ones(cfg.n_voxels).pin_memory()
    for _ in range(3):
        rec.reconstruct_host(evh, off, 1, fh.numpy())
    walls = []
    for _ in range(5):
        t = time.perf_counter()
        rec.reconstruct_host(evh, off, 1, fh.numpy())
        walls.append((time.perf_counter() - t) * 1e3)
    with profile(activities=[ProfilerActivity.CUDA]) as prof:
        t = time.perf_counter()
        rec.reconstruct_host(evh, off, 1, fh.numpy())
        wall = (time.perf_counter() - t) * 1e3
    rec.close()
    evs = []
    for e in prof.events():
        if e.device_type.name != "CUDA":
            continue
        evs.append((e.time_range.start, e.time_range.end, e.name))
    evs.sort()
    t0 = evs[0][0]
    rows = [(round((a - t0) / 1e3, 4), round((b - a) / 1e3, 4), n[:60]) for a, b, n in evs]
    kern = [r for r in rows if "k_" in r[2]]
    cp = [r for r in rows if "emcpy" in r[2] or "Memcpy" in r[2]]
    out = {"wall_ms": wall, "walls_unprofiled_ms": walls, "first_op_to_last_end_ms": (max(b for _, b, _ in evs) - t0) / 1e3,
           "first_kernel_start_ms": kern[0][0] if kern else None,
           "last_kernel_end_ms": max(r[0] + r[1] for r in kern) if kern else None,
           "kernel_busy_ms": sum(r[1] for r in kern), "copy_busy_ms": sum(r[1] for r in cp), "n_ops": len(rows)}
    print(json.dumps(out, indent=1))
    for r in rows[:40] + [("...",)] + rows[-30:]:
        print(*r, file=sys.stderr)


if __name__ == "__main__":
    main()
