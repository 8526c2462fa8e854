#!/usr/bin/env python
"""Offline analysis: L1->L2 *requests* per event under candidate 128-byte
line layouts of the 2x2x2-brick image. The projection's binding unit is the L1->XBAR request
interface (ncu: l1tex__m_l1tex2xbar_req_cycles_active ~79 %, ~1 request per SM clock), and
one request carries the sectors of one 128-byte line that a warp instruction touches.
Emulates the kernel's instruction grouping on the oracle's paths:
  - gathers: lane k takes dominant-axis slab k of a 32-slab round and issues three loads
    (the 1st, 2nd, 3rd piece of its slab); sectors already fetched for this LOR hit L1;
  - REDs: 32 consecutive path pieces per instruction (path order).
Analysis tooling, not product code; runs the oracle (test infrastructure).
Usage: python tests/analysis/request_sim.py [n_events] [config]"""
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import lmgen  # noqa: E402
import oracle  # noqa: E402

HALO = 2


def keys(ix, iy, iz, dims, line):
    """(sector id, line id) of voxels under 2x2x2-brick sectors and lines of
    line = (lx, ly, lz) bricks (lx*ly*lz = 4), lines laid out x-fastest."""
    px, py, pz = ix + HALO, iy + HALO, iz + HALO
    bx, by, bz = px >> 1, py >> 1, pz >> 1
    BX, BY = (dims[0] + 5) // 2, (dims[1] + 5) // 2
    lx, ly, lz = line
    if line == (4, 1, 1):  # the current layout: linear brick order, 4 consecutive bricks per line
        b = bx + BX * (by + BY * bz)
        return b, b >> 2
    LX, LY = -(-BX // lx), -(-BY // ly)
    ln = bx // lx + LX * (by // ly + LY * (bz // lz))
    sec = ln * 4 + (bx % lx) + lx * ((by % ly) + ly * (bz % lz))
    return sec, ln


def requests(sec, ln):
    """requests of one warp instruction: distinct lines among its sectors"""
    return len(np.unique(ln)), len(np.unique(sec))


def main():
    n = int(sys.argv[1]) if len(sys.argv) > 1 else 2000
    cfg = lmgen.CONFIGS[sys.argv[2] if len(sys.argv) > 2 else "C2"]
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    nx, ny, _ = cfg.dims
    ev = lmgen.subset_events(cfg, 0, n)
    lines = [(4, 1, 1), (2, 2, 1), (2, 1, 2), (1, 2, 2), (1, 4, 1), (1, 1, 4)]
    tot = {L: [0, 0, 0, 0] for L in lines}  # gather requests, gather sectors, RED requests, RED sectors
    pieces = 0
    for e in ev:
        co, _ = oracle.siddon_path(g, e[:3].astype(float), e[3:].astype(float))
        if len(co) == 0:
            continue
        ix, iy, iz = co % nx, (co // nx) % ny, co // (nx * ny)
        d = np.abs(e[3:] - e[:3]) / np.asarray(cfg.voxel_mm)
        dom = int(np.argmax(d))
        a = [ix, iy, iz][dom]
        # slab index along the dominant axis, in traversal order
        slab = np.abs(a - a[0])
        # rank of each piece within its slab (0, 1, 2)
        rank = np.zeros(len(co), int)
        for i in range(1, len(co)):
            rank[i] = rank[i - 1] + 1 if slab[i] == slab[i - 1] else 0
        pieces += len(co)
        for L in lines:
            sec, ln = keys(ix, iy, iz, cfg.dims, L)
            # gathers: per 32-slab round, three instructions (piece rank 0, 1, 2); L1 keeps
            # the sectors already fetched for this LOR
            seen = set()
            for r0 in range(0, int(slab.max()) + 1, 32):
                in_round = (slab >= r0) & (slab < r0 + 32)
                for t in range(3):
                    m = in_round & (rank == t)
                    if not m.any():
                        continue
                    s_new = [s for s in np.unique(sec[m]) if s not in seen]
                    if s_new:
                        s_new = np.asarray(s_new)
                        tot[L][0] += len(np.unique(s_new // 4 if L != (4, 1, 1) else s_new >> 2))
                        tot[L][1] += len(s_new)
                        seen.update(s_new.tolist())
            # REDs: 32 consecutive pieces per instruction
            for s0 in range(0, len(co), 32):
                rq, sc = requests(sec[s0:s0 + 32], ln[s0:s0 + 32])
                tot[L][2] += rq
                tot[L][3] += sc
    ne = len(ev)
    print(f"{cfg.name}: {ne} events, {pieces / ne:.1f} pieces per event")
    print("line (bricks x,y,z) | gather req/ev  sec/ev | RED req/ev  sec/ev | total req/ev")
    for L in lines:
        gq, gs, rq, rs = (v / ne for v in tot[L])
        print(f"{str(L):19s} | {gq:8.1f} {gs:8.1f} | {rq:8.1f} {rs:8.1f} | {gq + rq:8.1f}")


if __name__ == "__main__":
    main()
