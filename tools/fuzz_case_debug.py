#!/usr/bin/env python
"""Diagnostic: one fuzz case (tests/test_fuzz_gpu.py case(seed)) — the voxel with the largest
relative error after one subset step, its contributing events, and per event the GPU's and
the oracle's contribution a_ij / fp_i to that voxel (single-event error images).
Usage (GPU box): python tools/fuzz_case_debug.py SEED"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tests"))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import oracle  # noqa: E402
import paper_conf_ipps_steuwerkg12_b200 as pkg  # noqa: E402
from test_fuzz_gpu import case  # noqa: E402

seed = int(sys.argv[1])
dims, vox, ev, s, f0, slabs = case(seed)
g = oracle.geom(dims, vox)
V = int(np.prod(dims))
rec = pkg.Reconstructor(dims, vox, torch.from_numpy(s).cuda())
rec.set_slabs(slabs)
f = torch.from_numpy(f0).cuda()
rec.subset_step(torch.from_numpy(ev).cuda(), f)
rec.synchronize()
got = f.cpu().numpy().astype(np.float64)
ref = oracle.subset_step(g, ev, s, f0)
mm = ref > 1e-3 * ref.max()
rel = np.zeros(V)
rel[mm] = np.abs(got[mm] - ref[mm]) / ref[mm]
j = int(np.argmax(rel))
print("dims", dims, "vox", vox, "slabs", slabs, "worst voxel", j, np.unravel_index(j, dims[::-1]), "rel", rel[j],
      "f0", f0[j], "s", s[j], "ref", ref[j], "got", got[j])
fp_or = oracle.forward(g, ev, f0)
c_all = torch.empty(V, device="cuda")
rec.error_image(torch.from_numpy(ev).cuda(), torch.from_numpy(f0).cuda(), c_all)
c_ref = oracle.error_image(g, ev, f0)
print("c_j gpu", float(c_all[j]), "oracle", c_ref[j], "rel", abs(float(c_all[j]) - c_ref[j]) / c_ref[j])
rows = []
for i, e in enumerate(ev):
    co, ln = oracle.siddon_path(g, e[:3].astype(float), e[3:].astype(float))
    if j in set(co.tolist()) and fp_or[i] > 0:
        lj = float(ln[list(co).index(j)])
        one = torch.from_numpy(ev[i:i + 1]).cuda()
        c1 = torch.empty(V, device="cuda")
        rec.error_image(one, torch.from_numpy(f0).cuda(), c1)
        fpg = torch.empty(1, device="cuda")
        rec.forward(one, torch.from_numpy(f0).cuda(), fpg)
        rows.append((i, lj, len(co), fp_or[i], float(fpg[0]), lj / fp_or[i], float(c1[j])))
rows.sort(key=lambda r: -abs(r[6] - r[5]))
print("event  a_ij  path_len  fp_oracle  fp_gpu  contrib_oracle  contrib_gpu  rel_diff")
for r in rows[:15]:
    print(r[0], "%.3e" % r[1], r[2], "%.6e" % r[3], "%.6e" % r[4], "%.6e" % r[5], "%.6e" % r[6],
          "%.2e" % (abs(r[6] - r[5]) / max(r[5], 1e-30)), ev[r[0]])
rec.close()
