#!/usr/bin/env python
"""Projection time of a rank's share of a C2 subset (1/P of 10^6 events) on one B200: the
per-rank work of the P-GPU strong-scaling configuration C3 (diagnostic)."""
import json

import numpy as np
import torch

import lmgen
import paper_conf_ipps_steuwerkg12_b200 as pkg


def main():
    cfg = lmgen.CONFIGS["C2"]
    ev = torch.from_numpy(lmgen.subset_events(cfg, 0)).cuda()
    s = torch.from_numpy(lmgen.norm(cfg)).cuda()
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, s)
    f = torch.ones(cfg.n_voxels, device="cuda")
    out = {}
    for P in (1, 2, 4, 8, 16, 100, 1000):
        n = cfg.n_events // P
        off = np.array([0, n], np.int64)
        for _ in range(3):
            rec.reconstruct(ev[:n], off, 1, f)
        rec.synchronize()
        rec.set_timing(True)
        for _ in range(20):
            rec.reconstruct(ev[:n], off, 1, f)
        rec.synchronize()
        st = rec.stats()
        rec.set_timing(False)
        k = st["timed_subsets"]
        out[P] = {"events": n, "project_ms": st["project_ms"] / k, "update_ms": st["update_ms"] / k}
        out[P]["efficiency_vs_P1"] = (out[1]["project_ms"] / P) / out[P]["project_ms"]
        # fresh counters for the next size
        rec.close()
        rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, s)
    rec.close()
    print(json.dumps(out, indent=1))


if __name__ == "__main__":
    main()
