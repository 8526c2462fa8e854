"""Diagnostic for the fused combine on a 1-rank communicator."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch, lmgen
import paper_conf_ipps_steuwerkg12_b200 as pkg
cfg = lmgen.CONFIGS["C1"]; ev = torch.from_numpy(lmgen.subset_events(cfg, 0)).cuda()
s = torch.from_numpy(lmgen.norm(cfg)).cuda()
for mode in (2, 3):
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, s, dist=(0, 1, pkg.nccl_unique_id()))
    rec.set_combine(mode)
    f = torch.full((cfg.n_voxels,), 2.0, device="cuda")
    rec.subset_step(ev[:0], f); rec.synchronize()
    print("mode", mode, "no events: f mean", f.mean().item(), "min", f.min().item(), "max", f.max().item())
    f = torch.ones(cfg.n_voxels, device="cuda")
    rec.subset_step(ev, f); rec.synchronize()
    print("mode", mode, "events: f mean", f.mean().item(), "min", f.min().item(), "max", f.max().item(), rec.stats()["launches"])
    c = torch.empty(cfg.n_voxels, device="cuda"); rec.error_image(ev, torch.ones_like(f), c); rec.synchronize()
    print("   error image sum", c.sum().item())
    rec.close()
