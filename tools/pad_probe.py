"""Allocation-placement probe: the C5 (hot-spot) projection time against a dummy device
allocation made before lmosem_init, which shifts where the library's brick images land.
One process per (library, pad); prints ms per subset (reconstruct over the 10 subsets, x3)."""
import os
import sys
import time

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import lmgen  # noqa: E402
import paper_conf_ipps_steuwerkg12_b200 as pkg  # noqa: E402


def main(name, pad_mb):
    cfg = lmgen.CONFIGS[name]
    L, N = cfg.n_subsets, cfg.n_events
    ev = torch.from_numpy(lmgen.events(cfg, 0, N * L)).cuda()
    norm = torch.from_numpy(lmgen.norm(cfg)).cuda()
    f = torch.ones(cfg.n_voxels, device="cuda")
    pad = torch.empty(int(pad_mb * (1 << 20)) // 4 + 1, device="cuda")  # noqa: F841
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, norm, stream=torch.cuda.current_stream())
    offs = np.arange(L + 1, dtype=np.int64) * N
    rec.reconstruct(ev, offs, 1, f)
    torch.cuda.synchronize()
    best = 1e9
    for _ in range(3):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        rec.reconstruct(ev, offs, 3, f)
        b.record()
        torch.cuda.synchronize()
        best = min(best, a.elapsed_time(b) / (3 * L))
    print(f"{name} lib={os.environ.get('LMOSEM_LIB') or 'new'} pad={pad_mb} MB: {best:.4f} ms per subset", flush=True)
    rec.close()


if __name__ == "__main__":
    main(sys.argv[1], float(sys.argv[2]))
