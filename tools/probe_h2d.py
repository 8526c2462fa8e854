#!/usr/bin/env python
"""Pinned H2D / D2H bandwidth and the host path's phase times at C2 (diagnostic)."""
import json
import time

import numpy as np
import torch

import lmgen
import paper_conf_ipps_steuwerkg12_b200 as pkg


def bw(nbytes, d2h=False, reps=20):
    h = torch.empty(nbytes, dtype=torch.uint8).pin_memory()
    d = torch.empty(nbytes, dtype=torch.uint8, device="cuda")
    for _ in range(3):
        (h.copy_(d, non_blocking=True) if d2h else d.copy_(h, non_blocking=True))
    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    for _ in range(reps):
        (h.copy_(d, non_blocking=True) if d2h else d.copy_(h, non_blocking=True))
    b.record()
    torch.cuda.synchronize()
    return nbytes * reps / (a.elapsed_time(b) * 1e-3) / 1e9


def main():
    out = {"h2d_GBps_24MB": bw(24 << 20), "d2h_GBps_24MB": bw(24 << 20, True), "h2d_GBps_256MB": bw(256 << 20)}
    cfg = lmgen.CONFIGS["C2"]
    ev = lmgen.events(cfg, 0, cfg.n_events * cfg.n_subsets)
    s = lmgen.norm(cfg)
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, torch.from_numpy(s).cuda())
    evh = torch.from_numpy(ev).pin_memory()
    fh = torch.ones(cfg.n_voxels).pin_memory()
    for _ in range(2):
        rec.reconstruct_host(evh, off, 1, fh.numpy())
    rec.set_timing(True)
    walls = []
    for _ in range(5):
        t = time.perf_counter()
        rec.reconstruct_host(evh, off, 1, fh.numpy())
        walls.append(time.perf_counter() - t)
    out["wall_ms_per_recon"] = [w * 1e3 for w in walls]
    out["stats"] = rec.stats()
    rec.close()
    print(json.dumps(out))


if __name__ == "__main__":
    main()
