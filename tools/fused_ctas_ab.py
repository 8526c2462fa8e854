#!/usr/bin/env python
"""A/B (round 2): the fused combine launched with 4 / 2 / 1 CTAs per SM on a 1-rank communicator, in the reconstruction loop at a 1/8 share and a whole C2 subset, vs ALLREDUCE (plain update): does leaving SM room let the next projection start during the combine?"""
import os, sys, json
sys.path.insert(0, os.getcwd())
import numpy as np, torch, lmgen
import paper_conf_ipps_steuwerkg12_b200 as pkg
cfg = lmgen.CONFIGS["C2"]
L = 10
res = {}
for frac in (8, 1):
    n = cfg.n_events // frac
    ev = torch.from_numpy(lmgen.events(cfg, 0, n * L)).cuda()
    offs = np.arange(L + 1, dtype=np.int64) * n
    for mode in (1, 3):
        rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, torch.from_numpy(lmgen.norm(cfg)).cuda(), dist=(0, 1, pkg.nccl_unique_id()))
        rec.set_combine(mode)
        f = torch.ones(cfg.n_voxels, device="cuda")
        rec.reconstruct(ev, offs, 1, f); rec.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        st = torch.cuda.current_stream()
        a.record(st)
        rec.reconstruct(ev, offs, 5, f)
        b.record(st); torch.cuda.synchronize()
        res[f"1/{frac} mode{mode}"] = round(a.elapsed_time(b) / (5 * L), 4)
        rec.close()
print(os.environ.get("LMOSEM_FUSED_CTAS_PER_SM_AB", "4"), json.dumps(res))
