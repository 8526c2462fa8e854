#!/usr/bin/env python
"""torchrun worker of tests/test_nccl_multigpu.py (and a manual check on a multi-GPU node):
one process per GPU, NCCL communicator from a broadcast id, every combine of the library
(auto = fused multimem when its init self-test passed, else ISD; ALLREDUCE; ISD; FUSED) on a
C1 subset step, a C1 2-subset x 2-iteration reconstruction and a 200k-event C2 subset, each
against the float64 oracle on rank 0, with the f replicas of all ranks bitwise equal
(Listing 3). Rank 0 prints one JSON line with the results.
    python -m torch.distributed.run --nproc-per-node G --master-addr 127.0.0.1 tests/mp/nccl_parity_worker.py
"""
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402
import torch  # noqa: E402
import torch.distributed as dist  # noqa: E402

import lmgen  # noqa: E402
import paper_conf_ipps_steuwerkg12_b200 as pkg  # noqa: E402


def main():
    rank, world, local = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"]), int(os.environ["LOCAL_RANK"])
    torch.cuda.set_device(local)
    dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    os.environ.setdefault("LMOSEM_TIMEOUT_S", "120")
    cases = []
    c1 = lmgen.CONFIGS["C1"]
    ev1 = lmgen.events(c1, 0, c1.n_events * c1.n_subsets)
    off1 = np.arange(c1.n_subsets + 1) * c1.n_events
    c2 = lmgen.CONFIGS["C2"]
    ev2 = lmgen.subset_events(c2, 0, 200_000)
    results = {"world": world}
    for mode in (0, 1, 2, 3):
        for name, cfg, ev, off, iters in (("C1_subset", c1, ev1[:c1.n_events], None, 1),
                                          ("C1_recon", c1, ev1, off1, 2),
                                          ("C2_subset", c2, ev2, None, 1)):
            s = lmgen.norm(cfg)
            rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, torch.from_numpy(s).cuda(),
                                    dist=pkg.make_dist(rank, world))
            auto = rec.combine
            if mode:
                try:
                    rec.set_combine(mode)
                except pkg.LmosemError as e:
                    results[f"{name}_mode{mode}"] = {"unavailable": str(e)}
                    rec.close()
                    continue
            f = torch.ones(cfg.n_voxels, device="cuda")
            d_ev = torch.from_numpy(ev).cuda()
            if off is None:
                rec.subset_step(d_ev, f)
            else:
                rec.reconstruct(d_ev, off, iters, f)
            rec.synchronize()
            rec.close()
            allf = [torch.empty_like(f) for _ in range(world)]
            dist.all_gather(allf, f)
            if rank == 0:
                same = all(torch.equal(allf[0], x) for x in allf[1:])
                cases.append((name, mode, auto, cfg, ev, off, iters, s, allf[0].cpu().numpy(), same))
    if rank == 0:
        import oracle
        for name, mode, auto, cfg, ev, off, iters, s, got, same in cases:
            g = oracle.geom(cfg.dims, cfg.voxel_mm)
            f0 = np.ones(cfg.n_voxels)
            ref = oracle.subset_step(g, ev, s, f0) if off is None else oracle.reconstruct(g, ev, off, iters, s, f0)
            got = got.astype(np.float64)
            m = ref > 1e-3 * ref.max()
            results[f"{name}_mode{mode}"] = {
                "auto_combine": auto, "replicas_equal": bool(same),
                "max_rel": float(np.max(np.abs(got[m] - ref[m]) / ref[m])),
                "rel_l2": float(np.linalg.norm(got - ref) / np.linalg.norm(ref))}
        print(json.dumps(results), flush=True)
    dist.barrier()
    dist.destroy_process_group()


if __name__ == "__main__":
    main()
