#!/usr/bin/env python
"""compute-sanitizer target: a 2x10^4-event C2 subset step + sensitivity, fused and 3-slab."""
import numpy as np, torch, lmgen, paper_conf_ipps_steuwerkg12_b200 as pkg
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
    rec.synchronize(); rec.close()
print("ok")
