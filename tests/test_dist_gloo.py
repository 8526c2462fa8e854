"""Multi-process (world size 2 and 4, gloo, CPU) tests of the N > 1 host logic.

The GPU path's distribution (§IV.A) is: every rank
gets the whole subset, projects its block [floor(rN/P), floor((r+1)N/P)) (block
distribution, via the C ABI's lmosem_block_range), the per-rank error images are summed
by an all-reduce (copy(add)), and every rank applies the update to its replica. Here the
per-rank step 1 is the oracle and the all-reduce is gloo, so the decomposition and the
NCCL-id broadcast plumbing are checked without a GPU.
"""
import os
import socket

import numpy as np
import pytest

torch = pytest.importorskip("torch")
import torch.distributed as dist  # noqa: E402
import torch.multiprocessing as mp  # noqa: E402


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    import sys
    sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import lmgen
        import oracle
        import paper_conf_ipps_steuwerkg12_b200 as pkg
        oracle.set_threads(2)
        cfg = lmgen.CONFIGS["C1"]
        g = oracle.geom(cfg.dims, cfg.voxel_mm)
        ev = lmgen.subset_events(cfg, 0)
        s = lmgen.norm(cfg)
        f0 = np.random.default_rng(7).uniform(0.5, 2.0, cfg.n_voxels)
        # block distribution through the C ABI (host-only entry point)
        b, e = pkg.block_range(len(ev), rank, world)
        c = torch.from_numpy(oracle.error_image(g, ev[b:e], f0))
        dist.all_reduce(c)  # copy(add) combine
        f_dist = oracle.update(f0, c.numpy(), s)
        # every rank holds the same replica afterwards
        gathered = [torch.empty_like(c) for _ in range(world)]
        dist.all_gather(gathered, torch.from_numpy(f_dist))
        same = all(torch.equal(gathered[0], x) for x in gathered)
        f_one = oracle.subset_step(g, ev, s, f0)
        err = float(np.max(np.abs(f_dist - f_one) / f_one))
        # ISD step 2: rank r updates only its block of the image
        # from the summed c, then the blocks are all-gathered into the full f
        # blocks from the library's own ISD partition (lmosem_isd_block, host-only), here over
        # voxels instead of bricks: equal chunks of the padded allocation, the real part
        # updated by its owner, chunks all-gathered and the padding dropped
        V = cfg.n_voxels
        vb, ve, alloc = pkg.isd_block(V, rank, world)
        chunk = alloc // world
        f_block = torch.zeros(chunk, dtype=torch.float64)
        f_block[:ve - vb] = torch.from_numpy(oracle.update(f0[vb:ve], c.numpy()[vb:ve], s[vb:ve]))
        parts = [torch.empty(chunk, dtype=torch.float64) for _ in range(world)]
        dist.all_gather(parts, f_block)
        f_isd = torch.cat(parts).numpy()[:V]
        err = max(err, float(np.max(np.abs(f_isd - f_one) / f_one)))
        # NCCL-id broadcast plumbing used by the GPU path
        d = pkg.make_dist(rank, world)
        ids = [None] * world
        dist.all_gather_object(ids, d[2])
        q.put((rank, b, e, same, err, d[0], d[1], len(d[2]), all(x == ids[0] for x in ids)))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world", [2, 3, 4])
def test_psd_ranks_gloo(world):
    port = _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = sorted(q.get(timeout=240) for _ in range(world))
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    n = 10000
    for r, (rank, b, e, same, err, d_rank, d_world, id_len, ids_equal) in enumerate(res):
        assert rank == r and (b, e) == ((r * n) // world, ((r + 1) * n) // world)
        assert same and err <= 1e-12
        assert (d_rank, d_world, id_len) == (r, world, 128) and ids_equal
