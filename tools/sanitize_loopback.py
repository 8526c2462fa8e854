#!/usr/bin/env python
"""compute-sanitizer target for the multi-rank combine: P = 3 ranks of a loopback world on
one GPU (ALLREDUCE, ISD, FUSED: the collectives' loop kernels and the cooperative fused
combine body) on a C1 subset and a 2-subset reconstruction of an odd anisotropic volume,
plus the fused combine of a 1-rank NCCL communicator (window set-up + self-test)."""
import os
import sys
import threading

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import lmgen  # noqa: E402
import paper_conf_ipps_steuwerkg12_b200 as pkg  # noqa: E402


def world(P, dims, vox, s, ev, offs, combine):
    g = pkg.Loopback(P)
    recs = [pkg.Reconstructor(dims, vox, torch.from_numpy(s).cuda(), stream=torch.cuda.Stream(), loopback=(g, r))
            for r in range(P)]
    for r in recs:
        r.set_combine(combine)
    V = int(np.prod(dims))
    fs = [torch.ones(V, device="cuda") for _ in range(P)]
    d_ev = torch.from_numpy(ev).cuda()
    torch.cuda.synchronize()

    def work(r):
        recs[r].subset_step(d_ev[:offs[1]], fs[r])
        recs[r].reconstruct(d_ev, offs, 1, fs[r])
        recs[r].synchronize()
    th = [threading.Thread(target=work, args=(r,)) for r in range(P)]
    for t in th:
        t.start()
    for t in th:
        t.join()
    out = [f.cpu() for f in fs]
    assert all(torch.equal(out[0], o) for o in out[1:])
    for r in recs:
        r.close()
    g.close()


cfg = lmgen.CONFIGS["C1"]
ev = lmgen.events(cfg, 0, 4000)
for combine in (1, 2, 3):
    world(3, cfg.dims, cfg.voxel_mm, lmgen.norm(cfg), ev, np.array([0, 2000, 4000], np.int64), combine)
dims, vox = (17, 13, 9), (1.0, 0.75, 1.5)
rng = np.random.default_rng(5)
half = 0.5 * np.asarray(dims) * np.asarray(vox)
ev2 = np.concatenate([rng.uniform(-1.4, 1.4, (3000, 3)) * half, rng.uniform(-1.4, 1.4, (3000, 3)) * half],
                     1).astype(np.float32)
for combine in (2, 3):
    world(3, dims, vox, rng.uniform(0.5, 2, int(np.prod(dims))).astype(np.float32), ev2,
          np.array([0, 1500, 3000], np.int64), combine)
rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, torch.from_numpy(lmgen.norm(cfg)).cuda(),
                        dist=(0, 1, pkg.nccl_unique_id()))
rec.set_combine(3)
f = torch.ones(cfg.n_voxels, device="cuda")
rec.reconstruct(torch.from_numpy(ev).cuda(), np.array([0, 2000, 4000], np.int64), 1, f)
rec.synchronize()
rec.close()
print("ok")
