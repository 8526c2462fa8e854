#!/usr/bin/env python
"""Per-warp timeline of the fused projection (diagnostic): builds the LMK_TRACE=1 variant
(variants/liblmosem_trace.so, here on CPU: `python tools/trace_tail.py build`), then on the
GPU runs one C2 subset share of n events and reports, from %globaltimer stamps per warp,
the ramp (entry -> first LOR), the tail (spread of the warps' exit times) and claims."""
import ctypes
import json
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
OUT = os.environ.get("LMOSEM_TRACE_LIB") or os.path.join(ROOT, "variants", "liblmosem_trace.so")


def build():
    from paper_conf_ipps_steuwerkg12_b200 import build as b
    os.makedirs(os.path.dirname(OUT), exist_ok=True)
    b.build(defines=["LMK_TRACE=1"], out=OUT)
    print("built", OUT)


def run(shares):
    os.environ["LMOSEM_LIB"] = OUT
    import torch

    import lmgen
    import paper_conf_ipps_steuwerkg12_b200 as pkg
    lib = ctypes.CDLL(OUT)
    cfg = lmgen.CONFIGS["C2"]
    ev = torch.from_numpy(lmgen.subset_events(cfg, 0)).cuda()
    s = torch.from_numpy(lmgen.norm(cfg)).cuda()
    res = {}
    for P in shares:
        n = cfg.n_events // P
        rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, s)
        f = torch.ones(cfg.n_voxels, device="cuda")
        c = torch.empty(cfg.n_voxels, device="cuda")
        for _ in range(3):
            rec.error_image(ev[:n], f, c)
        rec.synchronize()
        lib.lmosem_debug_trace_reset()
        rec.error_image(ev[:n], f, c)
        rec.synchronize()
        buf = np.zeros(16384 * 5, np.uint64)
        lib.lmosem_debug_trace(buf.ctypes.data_as(ctypes.c_void_p), ctypes.c_size_t(buf.nbytes))
        t = buf.reshape(-1, 5).astype(np.int64)
        t = t[t[:, 2] > 0]
        t0 = t[:, 0].min()
        start, first, end = (t[:, 0] - t0) / 1e3, (t[:, 1] - t0) / 1e3, (t[:, 2] - t0) / 1e3  # us
        pct = lambda a: {q: round(float(np.percentile(a, q)), 2) for q in (0, 10, 50, 90, 100)}
        res[P] = {"events": n, "warps": int(len(t)), "span_us": round(float(end.max()), 2),
                  "start_us": pct(start), "first_lor_us": pct(first[t[:, 1] > 0]), "exit_us": pct(end),
                  "lors_per_warp": pct(t[:, 3]), "claims_per_warp": pct(t[:, 4])}
        rec.close()
        print(P, json.dumps(res[P]), flush=True)
    return res


if __name__ == "__main__":
    if sys.argv[1] == "build":
        build()
    else:
        run([int(x) for x in sys.argv[2:]] or [1, 8, 16])
