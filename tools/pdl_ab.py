#!/usr/bin/env python
"""A/B of programmatic dependent launch (LMOSEM_PDL=0/1, read at lmosem_init): time per
subset of lmosem_reconstruct over 10 C2 subsets of N/P events each (P = 1, 2, 4, 8, 16:
a rank's share at P GPUs, without the combine), CUDA events on the library's stream,
alternating the two settings (diagnostic)."""
import json
import os

import numpy as np
import torch

import lmgen
import paper_conf_ipps_steuwerkg12_b200 as pkg


def main():
    cfg = lmgen.CONFIGS[os.environ.get("CFG", "C2")]
    L, N = cfg.n_subsets, cfg.n_events
    ev = torch.from_numpy(lmgen.events(cfg, 0, N * L)).cuda()
    s = torch.from_numpy(lmgen.norm(cfg)).cuda()
    stream = torch.cuda.current_stream()
    reps = int(os.environ.get("REPS", "30"))
    out = {}
    for P in (1, 2, 4, 8, 16):
        n = N // P
        sub = torch.cat([ev[l * N:l * N + n] for l in range(L)])
        off = np.arange(L + 1, dtype=np.int64) * n
        res = {"0": [], "1": []}
        for rnd in range(3):
            for pdl in ("0", "1"):
                os.environ["LMOSEM_PDL"] = pdl
                rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, s, stream=stream)
                f = torch.ones(cfg.n_voxels, device="cuda")
                for _ in range(3):
                    rec.reconstruct(sub, off, 1, f)
                torch.cuda.synchronize()
                a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                a.record(stream)
                for _ in range(reps):
                    rec.reconstruct(sub, off, 1, f)
                b.record(stream)
                torch.cuda.synchronize()
                res[pdl].append(a.elapsed_time(b) / (reps * L))
                rec.close()
        out[P] = {"events": n, "ms_per_subset_pdl0": min(res["0"]), "ms_per_subset_pdl1": min(res["1"]),
                  "all": res}
        out[P]["gain"] = out[P]["ms_per_subset_pdl0"] / out[P]["ms_per_subset_pdl1"]
    print(json.dumps(out, indent=1))


if __name__ == "__main__":
    main()
