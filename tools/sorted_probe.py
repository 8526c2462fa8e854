#!/usr/bin/env python
"""Probe: does processing events in a spatially sorted order (by the z of the LOR midpoint)
give the projection enough L2 locality to run the fused single pass on an image that does
not fit L2 (C4), or more L1 hits at C2?  Times the projection of one subset in each order
and slab setting (diagnostic; the subset's result is order-independent up to fp32 atomics)."""
import json
import sys

import numpy as np
import torch

import lmgen
import paper_conf_ipps_steuwerkg12_b200 as pkg


def time_proj(rec, ev, f, reps=5):
    n = ev.shape[0]
    off = np.array([0, n], np.int64)
    rec.reconstruct(ev, off, 1, f)
    rec.synchronize()
    rec.set_timing(True)
    for _ in range(reps):
        rec.reconstruct(ev, off, 1, f)
    rec.synchronize()
    st = rec.stats()
    rec.set_timing(False)
    return st["project_ms"] / st["timed_subsets"]


def main():
    name = sys.argv[1] if len(sys.argv) > 1 else "C4"
    cfg = lmgen.CONFIGS[name]
    ev = torch.from_numpy(lmgen.subset_events(cfg, 0)).cuda()
    s = torch.from_numpy(lmgen.norm(cfg)).cuda()
    zmid = 0.5 * (ev[:, 2] + ev[:, 5])
    orders = {"file": None, "zmid": torch.argsort(zmid)}
    # z-mid bins of ~8 mm, directions mixed inside a bin by a per-event hash
    zb = torch.floor(zmid / 8.0).to(torch.int64)
    h = (torch.arange(ev.shape[0], device="cuda", dtype=torch.int64) * 2654435761) % 1000003
    orders["zbin8_hash"] = torch.argsort(zb * 2000000 + h)
    # z-mid then transverse azimuth bins (similar LORs next to each other)
    az = torch.atan2(ev[:, 4] - ev[:, 1], ev[:, 3] - ev[:, 0])
    ab = torch.floor((az + np.pi) / (2 * np.pi) * 16).to(torch.int64).clamp(0, 15)
    orders["zbin8_az16"] = torch.argsort(zb * 100 + ab)
    out = {}
    slab_settings = (0, 1) if name == "C4" else (0,)
    for key, perm in orders.items():
        e = ev if perm is None else ev[perm].contiguous()
        for sl in slab_settings:
            rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, s)
            if sl:
                rec.set_slabs(sl)
            f = torch.ones(cfg.n_voxels, device="cuda")
            ms = time_proj(rec, e, f)
            out[f"{key}/slabs={rec.slabs if not sl else sl}"] = round(ms, 3)
            rec.close()
            print(key, sl, ms, flush=True)
    print(json.dumps({"config": name, "events": int(ev.shape[0]), "project_ms": out}, indent=1))


if __name__ == "__main__":
    main()
