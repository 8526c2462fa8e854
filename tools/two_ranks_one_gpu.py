#!/usr/bin/env python
"""Probe: two ranks of one NCCL communicator on the same GPU (launched by torchrun with
--nproc-per-node 2, both on cuda:0). NCCL normally rejects duplicate devices; if it does
not, the P = 2 combines (ISD, ALLREDUCE, FUSED) are checked against the oracle."""
import json
import os
import sys

import numpy as np
import torch
import torch.distributed as dist

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import lmgen  # noqa: E402
import paper_conf_ipps_steuwerkg12_b200 as pkg  # noqa: E402


def main():
    rank, world = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
    torch.cuda.set_device(0)
    dist.init_process_group("gloo")
    cfg = lmgen.CONFIGS["C1"]
    ev = lmgen.events(cfg, 0, cfg.n_events * cfg.n_subsets)
    s = lmgen.norm(cfg)
    out = {"rank": rank}
    try:
        rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, torch.from_numpy(s).cuda(), dist=pkg.make_dist(rank, world))
    except Exception as e:  # noqa: BLE001
        out["init"] = f"failed: {e}"
        print(json.dumps(out), flush=True)
        return
    out["init"] = "ok"
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    for mode in (1, 2, 3):
        try:
            rec.set_combine(mode)
            f = torch.ones(cfg.n_voxels, device="cuda")
            rec.reconstruct(torch.from_numpy(ev).cuda(), off, 1, f)
            rec.synchronize()
            out[f"combine{mode}"] = f.cpu().numpy().astype(np.float64).tolist()[:0] or float(f.sum().item())
            np.save(f"/tmp/f_r{rank}_m{mode}.npy", f.cpu().numpy())
        except Exception as e:  # noqa: BLE001
            out[f"combine{mode}"] = f"failed: {e}"
    rec.close()
    print(json.dumps(out), flush=True)


if __name__ == "__main__":
    main()
