#!/usr/bin/env python
"""Per-subset cost of each combine form on a 1-rank NCCL communicator (one B200): what the
exchange step costs on the device apart from NVLink traffic — kernel launches, NCCL's
own copies, the fused kernel's barriers and re-zeroing — next to the plain update
(diagnostic)."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np
import torch

import lmgen
import paper_conf_ipps_steuwerkg12_b200 as pkg


def main():
    cfg = lmgen.CONFIGS["C2"]
    L, N = cfg.n_subsets, cfg.n_events
    ev = torch.from_numpy(lmgen.events(cfg, 0, N * L)).cuda()
    s = torch.from_numpy(lmgen.norm(cfg)).cuda()
    offs = np.arange(L + 1, dtype=np.int64) * N
    out = {}
    for name, mode in (("none", None), ("allreduce", 1), ("isd", 2), ("fused", 3)):
        dist = None if mode is None else (0, 1, pkg.nccl_unique_id())
        rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, s, dist=dist)
        if mode is not None:
            rec.set_combine(mode)
        f = torch.ones(cfg.n_voxels, device="cuda")
        rec.reconstruct(ev, offs, 1, f)
        rec.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        st = torch.cuda.current_stream()
        torch.cuda.synchronize()
        a.record(st)
        for _ in range(5):
            rec.reconstruct(ev, offs, 1, f)
        rec.synchronize()
        b.record(st)
        torch.cuda.synchronize()
        ms = a.elapsed_time(b) / (5 * L)
        rec.set_timing(True)
        for _ in range(3):
            rec.reconstruct(ev, offs, 1, f)
        stt = rec.stats()
        rec.set_timing(False)
        k = stt["timed_subsets"]
        out[name] = {"ms_per_subset": ms, "project_ms": stt["project_ms"] / k, "combine_ms": stt["combine_ms"] / k,
                     "update_ms": stt["update_ms"] / k, "combine_mode": rec.combine}
        rec.close()
        print(name, json.dumps(out[name]), flush=True)
    print(json.dumps(out, indent=1))


if __name__ == "__main__":
    main()
