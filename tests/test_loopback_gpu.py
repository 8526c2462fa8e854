"""The multi-GPU combine (NEXT-1) run on ONE GPU and checked against
the float64 oracle: P ranks of an emulated world (the loopback transport of
include/lmosem.h, "Emulated world") execute the library's real subset_iteration — the
block split of the events, the ISD brick chunks with their
nb_alloc padding, in-place reduce-scatter / all-gather offsets and the zero_to re-zeroing
(Listing 3 l.6, l.15-16), the all-reduce form, and the fused
one-kernel combine body — each rank from its own host thread, as P processes would.

Acceptance is the north_star bar (BASELINE.json): max rel <= 1e-4 after one subset,
relative L2 <= 1e-3 after a reconstruction; the f replicas of all ranks must be bitwise
equal (copy distribution).
"""
import threading

import numpy as np
import pytest

import lmgen
import oracle

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

MAXREL_SUBSET = 1e-4
REL_L2_RECON = 1e-3
WORLDS = (2, 3, 4, 8)
COMBINES = (1, 2, 3)  # ALLREDUCE, ISD, FUSED


@pytest.fixture(scope="module")
def pkg():
    if not torch.cuda.is_available():
        pytest.skip("needs a GPU")
    import paper_conf_ipps_steuwerkg12_b200 as p
    p.load()
    return p


def dev(a):
    return torch.from_numpy(np.ascontiguousarray(a)).cuda()


def maxrel(got, ref):
    m = ref > 1e-3 * ref.max()
    v = float(np.max(np.abs(got[m] - ref[m]) / ref[m]))
    print(f"[parity] max rel err {v:.3e} over {int(m.sum())} voxels")
    return v


def rel_l2(got, ref):
    v = float(np.linalg.norm(got - ref) / np.linalg.norm(ref))
    print(f"[parity] rel L2 err {v:.3e}")
    return v


def run_world(pkg, P, cfg, s, combine, call, f0=None, slabs=0):
    """Creates P loopback ranks (own stream each), runs call(rec, f) on every rank from its
    own thread, and returns the P f images (float64 numpy) plus each rank's stats. slabs > 0
    forces the z-slab form (the listed one by default) on every rank."""
    group = pkg.Loopback(P)
    recs, fs = [], []
    f0 = np.ones(cfg.n_voxels, np.float32) if f0 is None else f0.astype(np.float32)
    for r in range(P):
        rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), stream=torch.cuda.Stream(), loopback=(group, r))
        rec.set_combine(combine)
        rec.set_slabs(slabs)
        assert rec.combine == combine and rec.world == P and rec.rank == r
        recs.append(rec)
        fs.append(dev(f0))
    torch.cuda.synchronize()
    errs = [None] * P

    def worker(r):
        try:
            call(recs[r], fs[r])
            recs[r].synchronize()
        except Exception as e:  # noqa: BLE001 (re-raised below)
            errs[r] = e

    th = [threading.Thread(target=worker, args=(r,)) for r in range(P)]
    for t in th:
        t.start()
    for t in th:
        t.join(timeout=600)
    assert not any(t.is_alive() for t in th), "a rank hung"
    for e in errs:
        if e is not None:
            raise e
    out = [f.cpu().numpy() for f in fs]
    stats = [rec.stats() for rec in recs]
    for rec in recs:
        rec.close()
    group.close()
    for r in range(1, P):  # copy distribution: identical replicas
        assert np.array_equal(out[r], out[0]), f"rank {r} replica differs from rank 0"
    return out[0].astype(np.float64), stats


_cache = {}


def cached(key, fn):
    if key not in _cache:
        _cache[key] = fn()
    return _cache[key]


def c1():
    def mk():
        cfg = lmgen.CONFIGS["C1"]
        ev = lmgen.events(cfg, 0, cfg.n_events * cfg.n_subsets)
        return cfg, ev, lmgen.norm(cfg)
    return cached("C1", mk)


@pytest.mark.parametrize("combine", COMBINES)
@pytest.mark.parametrize("P", WORLDS)
def test_loopback_c1_subset_and_reconstruction(pkg, P, combine):
    """C1: one subset (max rel vs oracle.subset_step) and 2 subsets x 2 iterations (rel L2
    vs oracle.reconstruct) with P ranks; every rank projects only its block."""
    cfg, ev, s = c1()
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    ev0 = ev[:cfg.n_events]
    d_ev0 = dev(ev0)
    got, stats = run_world(pkg, P, cfg, s, combine, lambda rec, f: rec.subset_step(d_ev0, f))
    ref = cached(("C1", "subset"), lambda: oracle.subset_step(g, ev0, s, np.ones(cfg.n_voxels)))
    assert maxrel(got, ref) <= MAXREL_SUBSET
    assert sum(st["events"] for st in stats) == len(ev0)
    for r, st in enumerate(stats):
        b, e = pkg.block_range(len(ev0), r, P)
        assert st["events"] == e - b

    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    d_ev = dev(ev)
    got2, _ = run_world(pkg, P, cfg, s, combine, lambda rec, f: rec.reconstruct(d_ev, off, 2, f))
    ref2 = cached(("C1", "recon2"), lambda: oracle.reconstruct(g, ev, off, 2, s, np.ones(cfg.n_voxels)))
    assert rel_l2(got2, ref2) <= REL_L2_RECON


@pytest.mark.parametrize("combine", COMBINES)
@pytest.mark.parametrize("P,slabs", [(2, 2), (3, 3), (8, 2)])
def test_loopback_listed_zslab_form(pkg, P, slabs, combine):
    """The out-of-L2 step 1 (listed z-slab form: per-rank k_zclass lists of the rank's block,
    passes A/B and fused window launches) under P ranks and every combine: one C1 subset and
    2 subsets x 2 iterations against the oracle, replicas bitwise equal."""
    cfg, ev, s = c1()
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    ev0 = ev[:cfg.n_events]
    d_ev0 = dev(ev0)
    got, _ = run_world(pkg, P, cfg, s, combine, lambda rec, f: rec.subset_step(d_ev0, f), slabs=slabs)
    ref = cached(("C1", "subset"), lambda: oracle.subset_step(g, ev0, s, np.ones(cfg.n_voxels)))
    assert maxrel(got, ref) <= MAXREL_SUBSET
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    d_ev = dev(ev)
    got2, _ = run_world(pkg, P, cfg, s, combine, lambda rec, f: rec.reconstruct(d_ev, off, 2, f), slabs=slabs)
    ref2 = cached(("C1", "recon2"), lambda: oracle.reconstruct(g, ev, off, 2, s, np.ones(cfg.n_voxels)))
    assert rel_l2(got2, ref2) <= REL_L2_RECON


@pytest.mark.parametrize("combine", COMBINES)
@pytest.mark.parametrize("P", WORLDS)
def test_loopback_c2_reconstruction(pkg, P, combine):
    """configs[2] (C3) on one GPU: the paper-shaped 150x150x280 volume, 10 subsets x 10^6
    events block-distributed over P ranks, through lmosem_reconstruct; rel L2 vs the oracle
    after the reconstruction, and the one-subset bar after its first subset."""
    def mk():
        cfg = lmgen.CONFIGS["C2"]
        ev = lmgen.events(cfg, 0, cfg.n_events * cfg.n_subsets)
        s = lmgen.norm(cfg)
        g = oracle.geom(cfg.dims, cfg.voxel_mm)
        off = np.arange(cfg.n_subsets + 1) * cfg.n_events
        ref1 = oracle.subset_step(g, ev[:cfg.n_events], s, np.ones(cfg.n_voxels))
        ref = oracle.reconstruct(g, ev, off, 1, s, np.ones(cfg.n_voxels))
        return cfg, ev, s, off, ref1, ref, dev(ev)
    cfg, ev, s, off, ref1, ref, d_ev = cached("C2", mk)
    got1, _ = run_world(pkg, P, cfg, s, combine, lambda rec, f: rec.subset_step(d_ev[:cfg.n_events], f))
    assert maxrel(got1, ref1) <= MAXREL_SUBSET
    got, stats = run_world(pkg, P, cfg, s, combine, lambda rec, f: rec.reconstruct(d_ev, off, 1, f))
    assert rel_l2(got, ref) <= REL_L2_RECON
    assert maxrel(got, ref) <= 10 * MAXREL_SUBSET
    assert np.all(got > 0)
    assert all(st["subsets"] == cfg.n_subsets for st in stats)


@pytest.mark.parametrize("combine", COMBINES)
def test_loopback_ragged_and_empty_blocks(pkg, combine):
    """Fewer events than ranks (most blocks empty), an empty subset, and an odd volume
    whose brick count is not a multiple of P (padded ISD chunks, a short last chunk)."""
    P = 8
    cfg = lmgen.with_(lmgen.CONFIGS["C1"], n_events=5)
    ev = lmgen.events(cfg, 0, 5)
    s = lmgen.norm(cfg)
    got, _ = run_world(pkg, P, cfg, s, combine, lambda rec, f: rec.subset_step(dev(ev), f))
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev, s, np.ones(cfg.n_voxels))
    assert np.max(np.abs(got - ref) / ref) <= MAXREL_SUBSET
    empty = torch.empty(0, device="cuda")
    got0, _ = run_world(pkg, P, cfg, s, combine, lambda rec, f: rec.subset_step(empty, f))
    assert np.all(got0 == 1.0)

    dims, vox = (17, 13, 9), (1.0, 0.75, 1.5)
    g = oracle.geom(dims, vox)
    half = 0.5 * np.asarray(dims) * np.asarray(vox)
    rng = np.random.default_rng(11)
    n = 4000
    p1 = rng.uniform(-1.4, 1.4, (n, 3)) * half
    p2 = rng.uniform(-1.4, 1.4, (n, 3)) * half
    ev2 = np.concatenate([p1, p2], 1).astype(np.float32)
    V = int(np.prod(dims))
    s2 = rng.uniform(0.5, 2.0, V).astype(np.float32)
    f0 = rng.uniform(0.5, 2.0, V).astype(np.float32)
    cfg2 = lmgen.with_(lmgen.CONFIGS["C1"], dims=dims, voxel_mm=vox)
    for P in (3, 7):
        got2, _ = run_world(pkg, P, cfg2, s2, combine, lambda rec, f: rec.subset_step(dev(ev2), f), f0=f0)
        ref2 = oracle.subset_step(g, ev2, s2, f0.astype(np.float64))
        assert maxrel(got2, ref2) <= MAXREL_SUBSET


def test_loopback_world1_equals_single_gpu(pkg):
    """A 1-rank loopback world is the single-GPU path plus identity collectives."""
    cfg, ev, s = c1()
    ev0 = dev(ev[:cfg.n_events])
    for combine in COMBINES:
        got, _ = run_world(pkg, 1, cfg, s, combine, lambda rec, f: rec.subset_step(ev0, f))
        rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
        f = dev(np.ones(cfg.n_voxels, np.float32))
        rec.subset_step(ev0, f)
        rec.synchronize()
        rec.close()
        np.testing.assert_allclose(got, f.cpu().numpy(), rtol=1e-6, atol=0)


@pytest.mark.parametrize("P", (2, 3))
def test_loopback_sensitivity_allreduce(pkg, P):
    """lmosem_sensitivity is collective: block split + all-reduce of the back-projected
    ones; every rank gets the full image (oracle_sensitivity, pin P14)."""
    cfg, ev, s = c1()
    group = pkg.Loopback(P)
    recs = [pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), stream=torch.cuda.Stream(), loopback=(group, r))
            for r in range(P)]
    outs = [torch.empty(cfg.n_voxels, device="cuda") for _ in range(P)]
    d_ev = dev(ev[:cfg.n_events])
    torch.cuda.synchronize()
    th = [threading.Thread(target=lambda r=r: (recs[r].sensitivity(d_ev, outs[r]), recs[r].synchronize()))
          for r in range(P)]
    for t in th:
        t.start()
    for t in th:
        t.join(timeout=300)
    ref = oracle.sensitivity(oracle.geom(cfg.dims, cfg.voxel_mm), ev[:cfg.n_events])
    for r in range(P):
        got = outs[r].cpu().numpy().astype(np.float64)
        m = ref > 1e-3 * ref.max()
        assert np.max(np.abs(got[m] - ref[m]) / ref[m]) <= 1e-5
        assert np.array_equal(outs[r].cpu().numpy(), outs[0].cpu().numpy())
    for rec in recs:
        rec.close()
    group.close()


@pytest.mark.parametrize("combine", COMBINES)
def test_loopback_host_and_file_streaming(pkg, combine, tmp_path):
    """lmosem_reconstruct_host and lmosem_reconstruct_file at P = 3: each rank uploads /
    reads only its block of every subset; the result equals the oracle's."""
    cfg, ev, s = c1()
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    ref = cached(("C1", "recon1"), lambda: oracle.reconstruct(g, ev, off, 1, s, np.ones(cfg.n_voxels)))
    P = 3
    group = pkg.Loopback(P)
    recs = [pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), stream=torch.cuda.Stream(), loopback=(group, r))
            for r in range(P)]
    for rec in recs:
        rec.set_combine(combine)
    fh = [np.ones(cfg.n_voxels, np.float32) for _ in range(P)]
    path = str(tmp_path / "events.lm")
    np.ascontiguousarray(ev, np.float32).tofile(path)
    fd = [dev(np.ones(cfg.n_voxels, np.float32)) for _ in range(P)]
    torch.cuda.synchronize()

    def work(r):
        recs[r].reconstruct_host(ev, off, 1, fh[r])
        recs[r].reconstruct_file(path, off, 1, fd[r])
        recs[r].synchronize()
    th = [threading.Thread(target=work, args=(r,)) for r in range(P)]
    for t in th:
        t.start()
    for t in th:
        t.join(timeout=300)
    for r in range(P):
        assert np.array_equal(fh[r], fh[0])
        assert rel_l2(fh[r].astype(np.float64), ref) <= REL_L2_RECON
        assert rel_l2(fd[r].cpu().numpy().astype(np.float64), ref) <= REL_L2_RECON
    for rec in recs:
        rec.close()
    group.close()


def test_loopback_missing_rank_times_out(pkg, monkeypatch):
    """A rank that never reaches the collective: the others fail with ENCCL after
    LMOSEM_TIMEOUT_S instead of hanging, and their context then answers ESTATE."""
    import time
    monkeypatch.setenv("LMOSEM_TIMEOUT_S", "2")
    cfg, ev, s = c1()
    group = pkg.Loopback(2)
    recs = [pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), stream=torch.cuda.Stream(), loopback=(group, r))
            for r in range(2)]
    f = dev(np.ones(cfg.n_voxels, np.float32))
    t0 = time.time()
    with pytest.raises(pkg.LmosemError) as e:
        recs[0].subset_step(dev(ev[:cfg.n_events]), f)
    assert e.value.status == 4 and time.time() - t0 < 10  # ENCCL
    with pytest.raises(pkg.LmosemError) as e2:
        recs[0].synchronize()
    assert e2.value.status == 5  # ESTATE
    for rec in recs:
        rec.close()
    group.close()


def test_loopback_group_lifetime_and_arguments(pkg):
    cfg, ev, s = c1()
    group = pkg.Loopback(2)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), loopback=(group, 0))
    with pytest.raises(pkg.LmosemError):  # rank 0 taken
        pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), loopback=(group, 0))
    with pytest.raises(pkg.LmosemError):  # rank outside the world
        pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), loopback=(group, 2))
    with pytest.raises(pkg.LmosemError):  # a context is still registered
        group.close()
    rec.close()
    group.close()
