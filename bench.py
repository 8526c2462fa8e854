#!/usr/bin/env python
"""LM-OSEM subset-iteration benchmark (BASELINE.json metric: events/s per subset at the
paper's 150x150x280 shape; s/recon).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--impl lmosem|reference] [--config C2]

A step is one subset iteration (fused projection, c all-reduce when N > 1, update) of
one 10^6-event subset; steps cycle through the config's 10 subsets. Inputs (events,
norm, f) are resident in HBM before the timed region. The timed region is not flushed: the
events of the 10 subsets (240 MB at C2) exceed the 126 MB L2, f and c are the
reconstruction's persistent state; a second measurement flushes L2 (a 256 MB write)
before every step, outside the step's CUDA events (`flushed_subset_step`). Rank 0 prints
ONE JSON line.
N > 1 is launched by torchrun (one process per GPU, NCCL).

--impl reference times the float64 CPU oracle (the only reference this paper-only
workload has) on rank 0, each step a bounded sample of the same subset.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

import lmgen  # noqa: E402

METRIC = "LM-OSEM events/s per subset (150x150x280)"
# mean exact-Siddon path length per event (voxels) for the generated inputs
# (tools/path_stats.py, oracle on a 20k-event sample)
MEAN_PATH = {"C1": 25.37, "C2": 252.19, "C3": 252.19, "C4": 506.79, "C5": 440.96}
FLUSH_BYTES = 256 << 20
# NVLink 5 unidirectional GPU-to-GPU rate used to MODEL the combine's floor (t_AR,roof in
# SURVEY.md §8(d)); not measured here: every run of this repo has one GPU
NVLINK_GBS = 770.0
# The paper's own runtimes, as context only (Fig. 4b):
# the bar heights did not survive text extraction
PAPER_CONTEXT = {
    "what": "average runtime of one LM-OSEM subset iteration (~10^6 events, 150x150x280), SkelCL / OpenCL / CUDA "
            "on 1, 2 and 4 GPUs of a Tesla S1070 (GT200, 2009)",
    "value": "bar heights not recoverable; axis 0-4 s, so <= 4 s per subset on each bar",
    "relations": "CUDA about 20 % faster than OpenCL and SkelCL; SkelCL < 5 % overhead vs OpenCL",
    "cite": "PAPER.md lines 586-610, 655-675 (Fig. 4b)",
}


def env_int(k, d):
    return int(os.environ.get(k, d))


def parse():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=100)
    ap.add_argument("--warmup", type=int, default=5)
    ap.add_argument("--impl", default="lmosem", choices=["lmosem", "reference"])
    ap.add_argument("--config", default=None, help="C2 (N=1 default), C3 (N>1 default), C4, C5")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--cpu-sample", type=int, default=1_000_000,
                    help="events in cpu_baseline's timed oracle sample (C2: the whole subset, ~15 s of CPU work)")
    ap.add_argument("--ref-sample", type=int, default=200_000,
                    help="events per step of --impl reference (each step a bounded sample of the subset)")
    ap.add_argument("--slabs", type=int, default=0, help="z-slab passes for step 1 (0 = automatic)")
    ap.add_argument("--e2e-file", action="store_true",
                    help="also time lmosem_reconstruct_file from a raw list-mode file (page cache)")
    ap.add_argument("--combine", default="auto", choices=["auto", "allreduce", "isd", "fused"],
                    help="combine of the per-GPU error images for N > 1 (default: the library's auto mode, "
                         "fused when NVLS multimem is available and self-tested, else isd)")
    return ap.parse_args()


class ClockSampler:
    """nvidia-smi clocks + throttle reasons sampled every 200 ms during the timed region."""

    Q = ("clocks.sm,clocks.max.sm,clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
         "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, index: int):
        self.index = index
        self.proc = None
        self.lines = []

    def __enter__(self):
        try:
            self.proc = subprocess.Popen(["nvidia-smi", "-i", str(self.index), f"--query-gpu={self.Q}",
                                          "--format=csv,noheader,nounits", "-lms", "20"],
                                         stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
        except OSError:
            self.proc = None
        return self

    def _read(self):
        for line in self.proc.stdout:
            self.lines.append(line.strip())

    def __exit__(self, *a):
        if self.proc is not None:
            time.sleep(0.25)
            self.proc.terminate()
            try:
                self.proc.wait(timeout=5)
            except subprocess.TimeoutExpired:
                self.proc.kill()

    def summary(self):
        sm, mx, reasons = [], 0.0, set()
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        for ln in self.lines:
            p = [x.strip() for x in ln.split(",")]
            if len(p) < 6:
                continue
            try:
                sm.append(float(p[0]))
                mx = max(mx, float(p[1]))
            except ValueError:
                continue
            for n, v in zip(names, p[2:6]):
                if v.lower() == "active":
                    reasons.add(n)
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": mx or None,
                "reasons": sorted(reasons), "samples": len(sm)}


def measured_peaks():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as fh:
            return json.load(fh), "measured"
    except OSError:
        return {"hbm_gbs": 6650.0}, "fallback"


def l2_peak_gbs(V: int, nbf: int):
    """Live microbenchmark of random fp32 gather+RED pairs on a V-float buffer (the
    projection's L2 access mix); returns (pair ops/s, GB/s at 8 B per pair)."""
    import ctypes
    from paper_conf_ipps_steuwerkg12_b200 import build as b
    lib = ctypes.CDLL(b.L2PEAK_SO)
    lib.l2peak_run.argtypes = [ctypes.c_int, ctypes.c_int64, ctypes.c_int32, ctypes.POINTER(ctypes.c_float),
                               ctypes.POINTER(ctypes.c_double)]
    out = {}
    for name, mode in (("red", 0), ("ldg", 1), ("pair", 2), ("pair_run8", 4), ("pair_warp32", 5),
                       ("ldg_warp32", 7), ("red_warp32", 8)):
        ms, ops = ctypes.c_float(), ctypes.c_double()
        if lib.l2peak_run(mode, V, 256, ctypes.byref(ms), ctypes.byref(ops)) != 0:
            return None
        out[name] = ops.value / (ms.value * 1e-3)
    # the update's pattern (read 3 arrays, write 2, float4) over 3 arrays of nbf floats
    # each, 20 passes: elements/s (x 20 B = the streaming rate the update can reach)
    ms, ops = ctypes.c_float(), ctypes.c_double()
    if lib.l2peak_run(6, nbf, 20, ctypes.byref(ms), ctypes.byref(ops)) == 0:
        out["stream5_elems"] = ops.value / (ms.value * 1e-3)
    return out


def host_cores() -> int:
    try:
        return len(os.sched_getaffinity(0))
    except AttributeError:  # pragma: no cover
        return os.cpu_count() or 1


def cpu_model() -> str:
    try:
        with open("/proc/cpuinfo") as fh:
            for ln in fh:
                if ln.startswith("model name"):
                    return ln.split(":", 1)[1].strip()
    except OSError:
        pass
    return "unknown"


def cpu_baseline(cfg, sample: int):
    """The float64 oracle as it stands, on this host's cores, on a bounded sample."""
    import oracle
    oracle.set_threads(host_cores())  # all host cores (torchrun exports OMP_NUM_THREADS=1)
    ev = lmgen.subset_events(cfg, 0, sample)
    s = lmgen.norm(cfg)
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    f0 = np.ones(cfg.n_voxels)
    t0 = time.perf_counter()
    oracle.subset_step(g, ev, s, f0)
    dt = time.perf_counter() - t0
    s_subset = dt * cfg.n_events / sample  # one whole subset at this rate
    return {"value": sample / dt, "unit": "events/s", "cores": oracle.get_threads(), "kind": "oracle",
            "cpu_model": cpu_model(), "nproc": os.cpu_count(),
            "s_per_subset": s_subset, "s_per_recon": s_subset * cfg.n_subsets,
            "sample": f"{sample} events of subset 0 of {cfg.name} (one subset step incl. the {cfg.n_voxels}-voxel "
                      f"update), {dt:.2f} s wall, {dt * oracle.get_threads():.1f} core-s"}


def workload(cfg) -> str:
    """config.workload of both arms (the repo arm and --impl reference name the same workload)."""
    return (f"{cfg.name}: {cfg.note} LM-OSEM {cfg.dims[0]}x{cfg.dims[1]}x{cfg.dims[2]} @ {cfg.voxel_mm[0]} mm, "
            f"{cfg.n_subsets} subsets x {cfg.n_events} events, 1 iteration")


def padded_bricks(dims):
    """(bricks, real bricks) of the library's padded 2x2x2 brick image (halo 2 low, >= 2 high)."""
    B = [(d + 5) // 2 for d in dims]
    R = [(2 + d + 1) // 2 - 1 for d in dims]  # bricks [1, rhi) hold real voxels
    return B[0] * B[1] * B[2], R[0] * R[1] * R[2]


def combine_model(P: int, combine: str, dims) -> dict:
    """Modeled NVLink floor of the combine per subset (SURVEY.md §8(d) t_AR,roof(P)) at
    NVLINK_GBS per direction per GPU: all-reduce / ISD (reduce-scatter + all-gather) move
    2(P-1)/P |c| per GPU; the fused multimem kernel moves the real bricks' |c| each way
    (the switch pulls (P-1)/P of every rank's c, plus one multimem.st of the f block) —
    egress and ingress overlap in one pass."""
    nb, real = padded_bricks(dims)
    c_bytes = 32.0 * nb
    if P <= 1:
        return {"t_ms": 0.0, "bytes_per_gpu": 0.0}
    if combine == "fused":
        b = 32.0 * real
    else:
        b = 2.0 * (P - 1) / P * c_bytes
    return {"t_ms": b / (NVLINK_GBS * 1e9) * 1e3, "bytes_per_gpu": b, "nvlink_gbs": NVLINK_GBS,
            "what": f"modeled, not measured: {b / 1e6:.1f} MB per GPU at {NVLINK_GBS} GB/s ({combine})"}


def run_reference(args, cfg, rank):
    if rank != 0:
        return
    import oracle
    oracle.set_threads(host_cores())  # rank 0 alone runs: all host cores
    sample = min(args.ref_sample, cfg.n_events)
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    s = lmgen.norm(cfg)
    evs = [lmgen.subset_events(cfg, l % cfg.n_subsets, sample) for l in range(min(cfg.n_subsets, args.warmup + args.steps))]
    f = np.ones(cfg.n_voxels)
    for k in range(args.warmup):
        f = oracle.subset_step(g, evs[k % len(evs)], s, f)
    t0 = time.perf_counter()
    for k in range(args.steps):
        f = oracle.subset_step(g, evs[(args.warmup + k) % len(evs)], s, f)
    dt = time.perf_counter() - t0
    v = sample * args.steps / dt
    cores = oracle.get_threads()
    line = {"metric": METRIC, "value": v, "unit": "events/s", "impl": "reference", "n_gpus": args.gpus,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": 1e3 * dt / args.steps,
            "higher_is_better": True, "scaling": "strong", "vs_baseline": None, "dtype": "f64",
            "data": "synthetic", "config": {"workload": workload(cfg), "sample_events_per_step": sample,
                                            "sample": f"each oracle step runs a {sample}-event sample of the subset; "
                                                      f"value = sampled events / s"},
            "cpu_baseline": {"value": v, "unit": "events/s", "cores": cores, "kind": "oracle",
                             "cpu_model": cpu_model(), "nproc": os.cpu_count(),
                             "sample": f"{sample} events per step x {args.steps} steps"},
            "e2e": {"value": v, "unit": "events/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


def main():
    args = parse()
    world = env_int("WORLD_SIZE", 1)
    rank = env_int("RANK", 0)
    local = env_int("LOCAL_RANK", 0)
    name = args.config or ("C2" if world == 1 else "C3")
    cfg = lmgen.CONFIGS[name]
    if args.impl == "reference":
        return run_reference(args, cfg, rank)

    import torch
    import torch.distributed as dist

    import paper_conf_ipps_steuwerkg12_b200 as pkg

    torch.cuda.set_device(local)
    if world > 1:
        dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    dev = torch.device("cuda", local)

    # ---- inputs, resident in HBM (every rank holds the whole subsets; the library
    # projects its block: PAPER.md lines 503-505, block distribution)
    L = cfg.n_subsets
    ev_host = lmgen.events(cfg, 0, cfg.n_events * L)
    s_host = lmgen.norm(cfg)
    ev = torch.from_numpy(ev_host).to(dev)
    norm = torch.from_numpy(s_host).to(dev)
    f = torch.ones(cfg.n_voxels, device=dev)
    flush = torch.empty(FLUSH_BYTES // 4, device=dev)
    stream = torch.cuda.current_stream()
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, norm, dist=pkg.make_dist(rank, world), stream=stream)
    rec.set_slabs(args.slabs)
    if world > 1 and args.combine != "auto":
        rec.set_combine({"allreduce": 1, "isd": 2, "fused": 3}[args.combine])  # collective
    N = cfg.n_events

    def subset(k):
        l = k % L
        return ev[l * N:(l + 1) * N]

    offs = np.arange(L + 1, dtype=np.int64) * N

    def run_subsets(k0, count):
        """`count` subset iterations starting at subset k0 % L, as lmosem_reconstruct calls
        over consecutive subsets (a reconstruction's inner loop)."""
        calls = []
        while count > 0:
            l = k0 % L
            m = min(count, L - l)
            o = offs[l:l + m + 1] - offs[l]
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record(stream)
            rec.reconstruct(ev[offs[l]:offs[l + m]], o, 1, f)
            b.record(stream)
            calls.append((a, b, m))
            k0 += m
            count -= m
        return calls

    run_subsets(0, max(args.warmup, 3))
    rec.synchronize()

    # ---- timed region: K subset iterations of the reconstruction loop (lmosem_reconstruct
    # over the 10 subsets, cycling). L2 is not flushed: the events of the 10 subsets
    # (240 MB at C2) exceed the 126 MB L2; f and c are the algorithm's persistent state.
    # The library's per-phase CUDA events are OFF here (recording them between the kernels
    # costs ~14 us of GPU gaps per subset); an instrumented pass of the same loop right
    # after, inside the same clock-sampled window, gives the phase times and the
    # projection kernel's duration for the roofline.
    K = args.steps
    K2 = min(K, 50)
    launches0 = rec.stats()["launches"]
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    with ClockSampler(local) as clk:
        t_wall = time.perf_counter()
        calls = run_subsets(args.warmup, K)
        torch.cuda.synchronize()
        if world > 1:
            dist.barrier()
        t_wall = time.perf_counter() - t_wall
        launches = int(rec.stats()["launches"] - launches0)
        rec.set_timing(True)
        calls2 = run_subsets(args.warmup + K, K2)
        torch.cuda.synchronize()
        st = rec.stats()
        rec.set_timing(False)
    instr_ms = sum(a.elapsed_time(b) for a, b, _ in calls2) / K2
    per_call = [(a.elapsed_time(b), m) for a, b, m in calls]
    tot_ms = sum(t for t, _ in per_call)
    # per-subset time of each lmosem_reconstruct call (the paper reports the average per
    # subset; SURVEY.md §8(d) asks for the median beside it)
    med_ms = statistics.median(t / m for t, m in per_call)
    t = torch.tensor([tot_ms, st["convert_ms"], st["project_ms"], st["combine_ms"], st["update_ms"]], device=dev,
                     dtype=torch.float64)
    if world > 1:
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
    tot_ms, conv_ms, proj_ms, comb_ms, upd_ms = (float(x) for x in t.tolist())
    value = N * K / (tot_ms * 1e-3)  # events of the whole job (each subset's N split over ranks)
    # phase sums below are over the K2 instrumented steps
    conv_ms, proj_ms, comb_ms, upd_ms = (x / K2 for x in (conv_ms, proj_ms, comb_ms, upd_ms))

    # ---- secondary: single subset_step calls with L2 flushed before each (cold images)
    Kf = min(K, 20)
    fl = []
    for k in range(Kf):
        flush.fill_(float(k))
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(stream)
        rec.subset_step(subset(k), f)
        b.record(stream)
        fl.append((a, b))
    torch.cuda.synchronize()
    tf = torch.tensor([sum(a.elapsed_time(b) for a, b in fl)], device=dev, dtype=torch.float64)
    if world > 1:
        dist.all_reduce(tf, op=dist.ReduceOp.MAX)
    flushed = {"value": N * Kf / (float(tf.item()) * 1e-3), "unit": "events/s", "steps": Kf,
               "ms_per_step": float(tf.item()) / Kf,
               "what": "lmosem_subset_step per step (incl. the f -> brick conversion), 256 MB L2 flush before each "
                       "step outside its CUDA events"}

    # ---- per-rank share of a subset (N > 1 strong scaling: rank r projects N/P events of
    # every subset): the projection of the first N/P events of subset 0 on this GPU
    shares = None
    if world == 1:
        shares = {}
        for P in (2, 4, 8):
            n_p = N // P
            o = np.array([0, n_p], np.int64)
            rec.reconstruct(ev[:n_p], o, 1, f)
            rec.set_timing(True)
            for _ in range(10):
                rec.reconstruct(ev[:n_p], o, 1, f)
            stp = rec.stats()
            rec.set_timing(False)
            ms_p = stp["project_ms"] / stp["timed_subsets"]
            # the same share in the reconstruction loop (PDL chaining, no phase events):
            # 3 passes over L subsets of n_p events, projection + full update per subset
            offs_p = np.arange(L + 1, dtype=np.int64) * n_p
            rec.reconstruct(ev[:L * n_p], offs_p, 1, f)
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record(stream)
            rec.reconstruct(ev[:L * n_p], offs_p, 3, f)
            b.record(stream)
            torch.cuda.synchronize()
            loop_ms = a.elapsed_time(b) / (3 * L)
            shares[str(P)] = {"events": n_p, "project_ms": ms_p, "update_ms": stp["update_ms"] / stp["timed_subsets"],
                              "projection_efficiency": (proj_ms / P) / ms_p, "loop_ms_per_subset": loop_ms}
        shares["what"] = ("projection of 1/P of a subset (the per-rank step-1 work at P GPUs), CUDA events on the "
                          "library stream around the projection (they break the PDL overlap with the previous "
                          "kernel); projection_efficiency = (full-subset projection / P) / this; loop_ms_per_subset = "
                          "the same share as the reconstruction loop runs it (PDL chaining, no phase events): "
                          "projection + the FULL update per subset")

    # ---- e2e through the public API with HOST buffers: one host reconstruction over the
    # K subsets (pinned events streamed per subset, f uploaded and downloaded)
    e2e = None
    if not args.no_e2e:
        pinned = torch.from_numpy(ev_host).pin_memory()
        fh = torch.ones(cfg.n_voxels, dtype=torch.float32).pin_memory()  # pinned host image
        rec.reconstruct_host(pinned, offs[:2], 1, fh)  # warm-up (allocates the streaming buffers)
        reps = max(1, K // L)
        if world > 1:
            dist.barrier()
        rec.set_timing(True)  # copy-stream CUDA events around the event uploads (h2d_ms)
        t0 = time.perf_counter()
        for _ in range(reps):
            rec.reconstruct_host(pinned, offs, 1, fh)
        te = torch.tensor([time.perf_counter() - t0], dtype=torch.float64, device=dev)
        h2d_ms = rec.stats()["h2d_ms"]
        rec.set_timing(False)
        if world > 1:
            dist.all_reduce(te, op=dist.ReduceOp.MAX)
        b, e = pkg.block_range(N, rank, world)
        e2e = {"value": N * L * reps / float(te.item()), "unit": "events/s",
               "h2d_bytes_per_step": int(24 * (e - b) + 4 * cfg.n_voxels / L),
               "d2h_bytes_per_step": int(4 * cfg.n_voxels / L),
               "h2d_events_ms_per_subset": h2d_ms / (L * reps),
               "note": f"lmosem_reconstruct_host over {L} subsets x {reps} (pinned host events streamed per subset, "
                       f"overlapped with projection; pinned f H2D/D2H once per reconstruction), wall clock; "
                       f"h2d_events_ms_per_subset = the event uploads on the copy stream (the paper's phase 1), "
                       f"mostly hidden under the projection"}
        s_recon = float(te.item()) / reps
        if args.e2e_file:
            import tempfile
            with tempfile.TemporaryDirectory() as td:
                path = os.path.join(td, f"{name}_rank{rank}.lm")
                ev_host.tofile(path)
                fd_ = torch.ones(cfg.n_voxels, device=dev)
                rec.reconstruct_file(path, offs, 1, fd_)  # warm (page cache, staging buffers)
                torch.cuda.synchronize()
                t0 = time.perf_counter()
                for _ in range(reps):
                    rec.reconstruct_file(path, offs, 1, fd_)
                tfile = time.perf_counter() - t0
            e2e["file"] = {"value": N * L * reps / tfile, "unit": "events/s",
                           "what": "lmosem_reconstruct_file: raw list-mode file (page cache) -> pread into pinned "
                                   "double buffers -> H2D overlapped with projection; f on the device"}
    else:
        s_recon = None

    # every rank releases its context (NCCL communicator) together; rank 0 then runs the
    # single-GPU microbenchmarks and the oracle baseline and prints the line
    n_slabs, rec_combine = rec.slabs, rec.combine
    st_final = rec.stats()
    autotune = None
    if world > 1:  # the library timed the fused combine and ISD at init and kept the faster
        autotune = {"fused_ms": st_final["tune_fused_ms"], "isd_ms": st_final["tune_isd_ms"],
                    "allreduce_ms": st_final["tune_allreduce_ms"],
                    "chosen": {1: "allreduce", 2: "isd", 3: "fused"}.get(rec_combine),
                    "what": "ms per combine of each form, timed by lmosem_init on this box (max over ranks); "
                            "0 = the fused combine could not be set up or failed its self-test"}
    rec.close()
    if world > 1:
        dist.barrier()
        dist.destroy_process_group()
    if rank != 0:
        return

    peaks, peak_kind = measured_peaks()
    mean_path = MEAN_PATH[name]
    ev_per_launch = N / world
    pairs = ev_per_launch * mean_path
    proj_avg_s = proj_ms * 1e-3
    nbf = 8 * ((cfg.dims[0] + 5) // 2) * ((cfg.dims[1] + 5) // 2) * ((cfg.dims[2] + 5) // 2)  # padded bricks
    # the microbenchmarks run on a buffer of the size each projection launch works on: the
    # image (V floats), or in the z-slab form one slab of the brick image (L2-resident)
    l2_floats = cfg.n_voxels if n_slabs == 1 else nbf // n_slabs
    l2 = l2_peak_gbs(l2_floats, nbf)
    # the listed z-slab form (library default for images beyond L2: k_zclass lists, passes A/B
    # over the coarse slabs for the LORs that cross them, fused launches over fine windows)
    listed = n_slabs > 1 and os.environ.get("LMOSEM_ZLIST", "2") != "0"
    ev_reads = 1 if (n_slabs == 1 or listed) else 2 * n_slabs
    # 4 B gather + 4 B RED per path element, 24 B per event and read (the unlisted z-slab form
    # reads the events in each of its 2 x n_slabs launches; the listed form counts them once)
    alg_l2_bytes = pairs * 8.0 + ev_per_launch * 24.0 * ev_reads
    traffic, sectors, tr = None, None, None
    try:
        with open(os.path.join(ROOT, "profiles", "r02_traffic.json")) as fh:
            tr = json.load(fh).get(name)
        form_ok = tr and (tr.get("form") == "listed") == listed
        if form_ok and (listed or tr.get("launches_per_step", 1) == (2 * n_slabs if n_slabs > 1 else 1)):
            traffic = tr["dram_bytes_read_per_launch"] + tr["dram_bytes_write_per_launch"]
            sectors = tr["l2_sectors_read_per_launch"] + tr["l2_sectors_red_per_launch"]
    except (OSError, ValueError, KeyError):
        pass
    wide = ev_per_launch >= int(os.environ.get("LMOSEM_WIDE_N", "400000"))  # the library's MODE 6 rule
    kname = ((f"k_project<{6 if wide else 5}> (fused Siddon + forward + back-projection, texture gathers, "
              f"{'224 x 4' if wide else '256 x 3'} threads x CTAs per SM)") if n_slabs == 1 else
             (f"k_project<2,list>/<5,list>/<3,list> (listed z-slab form: k_zclass, then {n_slabs} forward-projection "
              f"launches over the LORs crossing each coarse slab, fused launches over overlapping fine windows for the "
              f"LORs inside one, {n_slabs} back-projection launches; summed per subset)") if listed else
             f"k_project<2>/<3> (z-slab form: {n_slabs} forward-projection + {n_slabs} back-projection launches per "
             f"subset, summed)")
    roof = {"kernel": kname, "bound": "l2",
            "achieved": alg_l2_bytes / proj_avg_s / 1e9, "unit": "GB/s", "traffic": traffic,
            "traffic_note": "DRAM bytes per launch, summed over one subset's launches in the z-slab form (ncu --set "
                            "full, profiles/r02_traffic.json); the algorithmic bytes are L2 traffic (the images, or "
                            "the slab being projected, stay L2-resident)",
            "per_unit": f"{mean_path} path elements x (4 B f gather + 4 B c RED) + 24 B event per event",
            "units_per_launch": ev_per_launch}
    if l2:
        roof["peak"] = l2["pair_warp32"] * 8.0 / 1e9
        roof["peak_kind"] = ("builder-measured live (libl2peak.so, not a driver number): fully coalesced fp32 gather+RED pairs (each warp on 32 consecutive "
                             f"floats) on a {l2_floats}-float L2-resident buffer (the image, or one z-slab of it; libl2peak.so, "
                             "PAIR_WARP32); the random-address pair rate is l2_micro_ops_per_s.pair")
        roof["frac"] = roof["achieved"] / roof["peak"]
        roof["frac_vs_random_pairs"] = roof["achieved"] / (l2["pair"] * 8.0 / 1e9)
        roof["l2_micro_ops_per_s"] = l2
    roof_sec = None
    if l2 and sectors and n_slabs > 1 and not listed:
        # z-slab form: the gathers (pass A) and the REDs (pass B) run in separate launches,
        # each bound by its own access type's sector rate -> a two-pass ceiling
        g_sec, r_sec = tr["l2_sectors_read_per_launch"], tr["l2_sectors_red_per_launch"]
        t_ceil = g_sec / l2["ldg"] + r_sec / l2["red"]
        roof_sec = {"bound": "l2_sectors_two_pass", "achieved": sectors / proj_avg_s, "peak": sectors / t_ceil,
                    "unit": "sectors/s", "frac": t_ceil / proj_avg_s, "sectors_per_launch": sectors,
                    "path_elements_per_sector": 2 * pairs / sectors,
                    "sector_overfetch": 32.0 * sectors / alg_l2_bytes,
                    "what": "ncu L2 sectors of one subset's z-slab launches (gathers in pass A, REDs in pass B) / live "
                            "projection time, vs the two-pass ceiling gathers / random-gather rate + REDs / random-RED "
                            "rate (live L2 microbenchmarks)"}
    elif l2 and sectors:
        # sector view: the L2 moves 32-byte sectors; both microbenchmarks (random and fully
        # coalesced gather+RED pairs) saturate at the same sector rate
        peak_sec = max(l2["red"], l2["ldg"], l2["pair"] * 2.0, l2["pair_run8"] * 2.0 / 8.0,
                       l2["pair_warp32"] * 2.0 / 8.0)
        roof_sec = {"bound": "l2_sectors", "achieved": sectors / proj_avg_s, "peak": peak_sec, "unit": "sectors/s",
                    "frac": sectors / proj_avg_s / peak_sec, "sectors_per_launch": sectors,
                    "path_elements_per_sector": 2 * pairs / sectors,
                    "sector_overfetch": 32.0 * sectors / alg_l2_bytes,
                    "what": "ncu L2 sectors of k_project (gathers + REDs, profiles/r02_traffic.json) / live duration, "
                            "vs the max sector rate over the live L2 microbenchmark modes (random RED, random gather, "
                            "random / 8-lane / 32-lane gather+RED pairs); sector_overfetch = 32 B x sectors / "
                            "algorithmic bytes (4 B gather + 4 B RED per path element, 24 B per event)"}
    # request view (DESIGN.md §7 summary): the SM->L2 request interface takes about one request
    # cycle per SM clock; a gather request (any sectors of one 128-byte line) costs one cycle,
    # a RED one cycle per 32-byte sector (tools/request_probe.cu)
    roof_req = None
    clocks = clk.summary()
    if sectors and tr and tr.get("l2_requests_read_per_launch"):
        sm_hz = (clocks.get("sm_mhz") or peaks.get("sm_max_mhz") or 1965.0) * 1e6
        cyc = tr["l2_requests_read_per_launch"] + tr["l2_sectors_red_per_launch"]
        peak_req = torch.cuda.get_device_properties(dev).multi_processor_count * sm_hz
        roof_req = {"bound": "l2_request_interface", "achieved": cyc / proj_avg_s, "peak": peak_req,
                    "unit": "request cycles/s", "frac": cyc / proj_avg_s / peak_req,
                    "request_cycles_per_launch": cyc, "ncu_req_cycles_active_pct": tr.get("req_cycles_active_pct"),
                    "what": "(gather requests + RED sectors) per launch (ncu, profiles/r02_traffic.json; summed over "
                            "a subset's launches in the z-slab form) / live duration, vs one request cycle per SM "
                            "clock (SMs x median SM clock under load)"}
    hbm = {"bound": "hbm", "achieved": (ev_per_launch * 24.0 * ev_reads) / proj_avg_s / 1e9,
           "peak": peaks["hbm_gbs"],
           "unit": "GB/s", "peak_kind": peak_kind, "what": "event streaming of k_project (24 B/event)"}
    hbm["frac"] = hbm["achieved"] / hbm["peak"]
    # k_update per step: read fb, c, s and write fb, c over the padded brick image (20 B per
    # voxel); the caller's f (4 B per voxel) is written once per reconstruction (1/L steps)
    upd_bytes = 20.0 * nbf + 4.0 * cfg.n_voxels / L
    upd = {"achieved": upd_bytes / (upd_ms * 1e-3) / 1e9, "unit": "GB/s",
           "what": f"k_update (20 B per padded voxel, {nbf} voxels, + the caller's f once per reconstruction)"}
    if l2 and "stream5_elems" in l2 and 12.0 * nbf < 100e6:
        # fb, c, s (12 B per voxel) stay L2-resident between projection and update
        upd.update({"bound": "l2", "peak": l2["stream5_elems"] * 20.0 / 1e9,
                    "peak_kind": "measured live: the update's read-3/write-2 float4 pattern streamed over three "
                                 "L2-resident nbf-float arrays (libl2peak.so, STREAM5)"})
    else:
        upd.update({"bound": "hbm", "peak": peaks["hbm_gbs"], "peak_kind": peak_kind})
    upd["frac"] = upd["achieved"] / upd["peak"]

    # whole-step roofline: t_roof = projection at the L2 pair peak + the
    # combine's modeled NVLink floor + the update at its streaming peak (1/P of it for the
    # ISD / fused combines), against the measured time per subset
    comb_name = {1: "allreduce", 2: "isd", 3: "fused"}.get(rec_combine, "allreduce") if world > 1 else "none"
    step_roof = None
    if l2:
        proj_roof_ms = alg_l2_bytes / (roof["peak"] * 1e9) * 1e3
        upd_roof_ms = upd_bytes / (upd["peak"] * 1e9) * 1e3 / (world if comb_name in ("isd", "fused") else 1)
        ar = combine_model(world, comb_name, cfg.dims)
        t_roof = proj_roof_ms + ar["t_ms"] + upd_roof_ms
        step_roof = {"t_roof_ms": t_roof, "t_meas_ms": tot_ms / K, "frac": t_roof / (tot_ms / K),
                     "terms_ms": {"project": proj_roof_ms, "combine_t_ar_roof": ar["t_ms"], "update": upd_roof_ms},
                     "combine_model": ar,
                     "what": "t_roof = projection bytes / live L2 pair peak + modeled NVLink floor of the combine + "
                             "update bytes / live streaming peak (/P for isd/fused); frac = t_roof / measured ms per "
                             "subset (whole job)"}
    share_model = None
    if shares:
        # the step one rank of 8 would run (C3 at P = 8), from the measured 1/8-share projection
        # and update on this GPU plus the modeled NVLink floor of the fused / ISD combine
        t1 = tot_ms / K
        share_model = {"P": 8, "t1_ms": t1, "project_share_ms": shares["8"]["project_ms"],
                       "update_share_ms": upd_ms / 8, "loop_share_ms": shares["8"]["loop_ms_per_subset"]}
        for cname in ("fused", "isd"):
            ar8 = combine_model(8, cname, cfg.dims)
            t8 = shares["8"]["project_ms"] + upd_ms / 8 + ar8["t_ms"]
            t8l = shares["8"]["loop_ms_per_subset"] - upd_ms * 7 / 8 + ar8["t_ms"]
            share_model[cname] = {"combine_roof_ms": ar8["t_ms"], "step_ms": t8, "efficiency_model": t1 / (8 * t8),
                                  "step_ms_loop": t8l, "efficiency_model_loop": t1 / (8 * t8l)}
        share_model["what"] = ("modeled P = 8 step from one GPU: the 1/8-share projection (CUDA events around it; or "
                               "_loop: the share's reconstruction loop, PDL on, minus 7/8 of the measured update) + 1/8 "
                               "of the measured update + the combine's modeled NVLink floor (770 GB/s); "
                               "efficiency_model = T1 / (8 T8). A model, not a multi-GPU measurement.")

    line = {
        "metric": METRIC, "value": value, "unit": "events/s", "n_gpus": world, "steps": K, "warmup": args.warmup,
        "ms_per_step": tot_ms / K, "ms_per_step_median": med_ms, "higher_is_better": True, "scaling": "strong", "vs_baseline": None,
        "dtype": "f32", "geometry_dtype": "f64", "data": "synthetic",
        "config": {"workload": workload(cfg),
                   "events_per_subset": N, "subsets": L, "parallelism": f"psd{world} (events block-distributed, f copy-distributed, c combined over NCCL)",
                   "l2": "not flushed: inputs larger than L2 (events of the 10 subsets, 24 B x N x 10); f, c "
                         "are the reconstruction's persistent state (flushed variant: flushed_subset_step)",
                   "z_slabs": n_slabs, "combine": {0: "none", 1: "allreduce", 2: "isd", 3: "fused"}.get(
                       rec_combine if world > 1 else 0)},
        "s_per_recon": tot_ms / K * L * 1e-3, "s_per_recon_e2e": s_recon,
        "timed_region": f"{K} subset iterations = lmosem_reconstruct calls over the {L} subsets, cycling; "
                        "CUDA events around each call on the library's stream; ms_per_step_median = median over the calls of "
                        "their per-subset time",
        "phase_ms_per_step": {"convert_f": conv_ms, "project": proj_ms, "combine": comb_ms, "update": upd_ms,
                              "steps": K2, "ms_per_step_instrumented": instr_ms,
                              "what": "library CUDA events around each phase on its stream, in an instrumented pass "
                                      "of the same loop right after the timed region"},
        "roofline": roof, "roofline_l2_sectors": roof_sec, "roofline_l2_requests": roof_req,
        "roofline_hbm_events": hbm, "roofline_update": upd, "roofline_step": step_roof,
        "combine_autotune": autotune,
        "p8_share_model": share_model,
        "gpu_launches": launches, "flushed_subset_step": flushed, "per_rank_share": shares,
        "clocks": clocks, "wall_s_timed_region": t_wall,
        "e2e": e2e,
        "paper_context": PAPER_CONTEXT,
    }
    if not args.no_cpu_baseline:  # rank 0 at every N
        line["cpu_baseline"] = cpu_baseline(cfg, min(args.cpu_sample, N))
    print(json.dumps(line), flush=True)


if __name__ == "__main__":
    main()
