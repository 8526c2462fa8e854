#!/usr/bin/env python
"""compute-sanitizer target: a 2x10^4-event C2 subset step + sensitivity, fused and 3-slab,
and a 3-subset reconstruction (the programmatic-dependent-launch chain project -> update ->
project)."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch, lmgen, paper_conf_ipps_steuwerkg12_b200 as pkg  # noqa: E401,E402
cfg = lmgen.CONFIGS["C2"]
ev = lmgen.subset_events(cfg, 0, 20000)
s = lmgen.norm(cfg)
for slabs in (0, 3):
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, torch.from_numpy(s).cuda())
    rec.set_slabs(slabs)
    f = torch.ones(cfg.n_voxels, device="cuda")
    rec.subset_step(torch.from_numpy(ev).cuda(), f)
    sens = torch.empty(cfg.n_voxels, device="cuda")
    rec.sensitivity(torch.from_numpy(ev).cuda(), sens)
    evr = torch.from_numpy(lmgen.events(cfg, 0, 30000)).cuda()
    rec.reconstruct(evr, np.array([0, 10000, 20000, 30000], np.int64), 1, f)
    rec.synchronize(); rec.close()
print("ok")
