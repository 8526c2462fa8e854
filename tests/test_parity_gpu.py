"""GPU parity: the CUDA path (through the C ABI) against the float64 oracle.

Acceptance (BASELINE.json north_star):
  - after one subset: max |f_gpu - f_or| / f_or <= 1e-4 over voxels with f_or > 1e-3 max f_or;
  - after a full reconstruction: ||f_gpu - f_or||_2 / ||f_or||_2 <= 1e-3.
Only the ordering of fp32 atomics (and fp32 rounding) may differ.
"""
import numpy as np
import pytest

import lmgen
import oracle
from conftest import GOLDEN, read_golden_paths

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

MAXREL_SUBSET = 1e-4
REL_L2_RECON = 1e-3


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


_cache = {}


def inputs(name, n_events=None):
    key = (name, n_events)
    if key not in _cache:
        cfg = lmgen.CONFIGS[name]
        if n_events is not None:
            cfg = lmgen.with_(cfg, n_events=n_events)
        ev = lmgen.events(cfg, 0, cfg.n_events * cfg.n_subsets)
        _cache[key] = (cfg, ev, lmgen.norm(cfg))
    return _cache[key]


def gpu_subset(pkg, cfg, ev, s, f0):
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    f = dev(f0.astype(np.float32))
    rec.subset_step(dev(ev), f)
    rec.synchronize()
    out = f.cpu().numpy().astype(np.float64)
    rec.close()
    return out


# ------------------------------------------------------------------ golden / edge cases
def test_golden_paths_on_gpu(pkg):
    """Hand-derived paths (tests/golden/paths_4cube.txt), incl. corner/face ties: with
    f = 1 the error image of one event is c_j = a_ij / sum_j a_ij, so c * chord = a_ij."""
    rec = pkg.Reconstructor((4, 4, 4), (1, 1, 1), dev(np.ones(64, np.float32)))
    f = dev(np.ones(64, np.float32))
    for name, p1, p2, pairs in read_golden_paths():
        ev = dev(np.array([p1 + p2], np.float32))
        c = torch.empty(64, device="cuda")
        rec.error_image(ev, f, c)
        fp = torch.empty(1, device="cuda")
        rec.forward(ev, f, fp)
        c = c.cpu().numpy().astype(np.float64)
        chord = sum(l for _, l in pairs)
        assert abs(fp.item() - chord) <= 1e-5 * max(chord, 1), name
        exp = np.zeros(64)
        for j, l in pairs:
            exp[j] = l / chord if chord > 0 else 0
        np.testing.assert_allclose(c, exp, rtol=2e-6, atol=1e-7, err_msg=name)
    rec.close()


def test_golden_em_update_on_gpu(pkg):
    cases = {c[0]: c for c in read_golden_paths()}
    ev = np.array([cases["G1"][1] + cases["G1"][2], cases["G2"][1] + cases["G2"][2]], np.float32)
    line = [l for l in open(f"{GOLDEN}/em_4cube.txt") if l.strip() and not l.startswith("#")][0]
    exp = np.ones(64)
    for tok in line.split():
        j, v = tok.split(":")
        exp[int(j)] = float(v)
    got = gpu_subset(pkg, lmgen.with_(lmgen.CONFIGS["C1"], dims=(4, 4, 4), voxel_mm=(1, 1, 1)), ev,
                     np.ones(64, np.float32), np.ones(64))
    np.testing.assert_allclose(got, exp, rtol=1e-6)


def test_degenerate_and_empty(pkg):
    cfg = lmgen.CONFIGS["C1"]
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(np.ones(cfg.n_voxels, np.float32)))
    f = dev(np.full(cfg.n_voxels, 2.0, np.float32))
    nan = float("nan")
    ev = np.array([[0, 0, 0, 0, 0, 0], [30, 30, 30, 40, 40, 40], [nan, 0, 0, 1, 1, 1],
                   [0, 0, float("inf"), 1, 1, 1], [-20, 8, 0, 20, 8, 0]], np.float32)
    rec.subset_step(dev(ev), f)
    rec.subset_step(torch.empty(0, 6, device="cuda"), f)  # empty subset: f unchanged
    rec.synchronize()
    assert torch.all(f == 2.0).item()
    rec.close()


def test_axis_parallel_lors(pkg):
    """LORs exactly parallel to one or two axes (zero direction components)."""
    cfg = lmgen.CONFIGS["C1"]
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    rng = np.random.default_rng(0)
    ev = []
    for k in range(300):
        p = rng.uniform(-7.9, 7.9, 3)
        q = p.copy()
        axes = [k % 3] if k % 2 else [k % 3, (k + 1) % 3]
        for a in axes:
            p[a], q[a] = -12.0, 12.0
        ev.append(np.concatenate([p, q]))
    ev = np.array(ev, np.float32)
    f0 = rng.uniform(0.5, 2.0, cfg.n_voxels)
    s = lmgen.norm(cfg)
    got = gpu_subset(pkg, cfg, ev, s, f0)
    ref = oracle.subset_step(g, ev, s, f0.astype(np.float32))
    assert maxrel(got, ref) <= MAXREL_SUBSET


# ------------------------------------------------------------------ C1 (configs[0])
def test_c1_forward_matches_oracle(pkg):
    cfg, ev, s = inputs("C1")
    rng = np.random.default_rng(1)
    f0 = rng.uniform(0.5, 2.0, cfg.n_voxels).astype(np.float32)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    fp = torch.empty(len(ev), device="cuda")
    rec.forward(dev(ev), dev(f0), fp)
    rec.synchronize()
    ref = oracle.forward(oracle.geom(cfg.dims, cfg.voxel_mm), ev, f0)
    got = fp.cpu().numpy()
    assert np.all((ref > 0) == (got > 0))
    m = ref > 0
    assert np.max(np.abs(got[m] - ref[m]) / ref[m]) <= 2e-6
    rec.close()


def test_c1_error_image_matches_oracle(pkg):
    cfg, ev, s = inputs("C1")
    f0 = np.random.default_rng(2).uniform(0.5, 2.0, cfg.n_voxels).astype(np.float32)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    c = torch.empty(cfg.n_voxels, device="cuda")
    rec.error_image(dev(ev[:cfg.n_events]), dev(f0), c)
    rec.synchronize()
    ref = oracle.error_image(oracle.geom(cfg.dims, cfg.voxel_mm), ev[:cfg.n_events], f0)
    got = c.cpu().numpy()
    assert np.all((ref > 0) == (got > 0))
    m = ref > 1e-3 * ref.max()
    assert np.max(np.abs(got[m] - ref[m]) / ref[m]) <= 1e-5
    rec.close()


def test_c1_one_subset(pkg):
    cfg, ev, s = inputs("C1")
    f0 = np.ones(cfg.n_voxels)
    got = gpu_subset(pkg, cfg, ev[:cfg.n_events], s, f0)
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev[:cfg.n_events], s, f0)
    assert maxrel(got, ref) <= MAXREL_SUBSET


def test_c1_listing2_literal_mode(pkg):
    """s = 1: Listing 2 exactly (f_j *= c_j where c_j > 0)."""
    cfg, ev, _ = inputs("C1")
    s = np.ones(cfg.n_voxels, np.float32)
    f0 = np.random.default_rng(3).uniform(0.5, 1.5, cfg.n_voxels)
    got = gpu_subset(pkg, cfg, ev[:cfg.n_events], s, f0)
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev[:cfg.n_events], s, f0.astype(np.float32))
    assert maxrel(got, ref) <= MAXREL_SUBSET


@pytest.mark.parametrize("iters", [1, 3])
def test_c1_full_reconstruction(pkg, iters):
    cfg, ev, s = inputs("C1")
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.reconstruct(dev(ev), off, iters, f)
    rec.synchronize()
    got = f.cpu().numpy().astype(np.float64)
    ref = oracle.reconstruct(oracle.geom(cfg.dims, cfg.voxel_mm), ev, off, iters, s, np.ones(cfg.n_voxels))
    assert rel_l2(got, ref) <= REL_L2_RECON
    assert np.all(got > 0)
    st = rec.stats()
    # one f -> brick conversion, then (project, update) per subset
    assert st["subsets"] == iters * cfg.n_subsets and st["launches"] == 2 * iters * cfg.n_subsets + 1
    rec.close()


def test_c1_host_reconstruct_matches_device(pkg):
    cfg, ev, s = inputs("C1")
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    fd = dev(np.ones(cfg.n_voxels, np.float32))
    rec.reconstruct(dev(ev), off, 2, fd)
    rec.synchronize()
    fh = np.ones(cfg.n_voxels, np.float32)
    evh = torch.from_numpy(ev).pin_memory()
    rec.reconstruct_host(evh, off, 2, fh)
    np.testing.assert_allclose(fh, fd.cpu().numpy(), rtol=1e-5)
    rec.close()


@pytest.mark.parametrize("slabs", [0, 3])
def test_c2_host_reconstruct_pipelined(pkg, slabs):
    """C2-sized host path: the first subset's upload is chunked (projected as the chunks
    land) and the final f is downloaded per brick z-range as the update finishes; the
    result is the oracle's 2-subset reconstruction (rel L2) and equals the device path's."""
    cfg = lmgen.CONFIGS["C2"]
    L = 2
    ev = lmgen.events(cfg, 0, cfg.n_events * L)
    s = lmgen.norm(cfg)
    off = np.arange(L + 1) * cfg.n_events
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    rec.set_slabs(slabs)
    f0 = np.random.default_rng(21).uniform(0.5, 2.0, cfg.n_voxels).astype(np.float32)
    fh = f0.copy()
    rec.reconstruct_host(torch.from_numpy(ev).pin_memory(), off, 1, fh)
    fd = dev(f0)
    rec.reconstruct(dev(ev), off, 1, fd)
    rec.synchronize()
    rec.close()
    assert maxrel(fh.astype(np.float64), fd.cpu().numpy().astype(np.float64)) <= 1e-5
    ref = oracle.reconstruct(oracle.geom(cfg.dims, cfg.voxel_mm), ev, off, 1, s, f0.astype(np.float64))
    assert rel_l2(fh.astype(np.float64), ref) <= REL_L2_RECON
    assert maxrel(fh.astype(np.float64), ref) <= 2 * MAXREL_SUBSET


def test_emulated_psd_ranks(pkg):
    """PAPER.md §IV.A (lines 476-485): summing the error images of the P blocks of a
    subset (each computed separately, as P ranks would) equals the whole subset's."""
    cfg, ev, s = inputs("C1")
    ev = ev[:cfg.n_events]
    f0 = dev(np.random.default_rng(4).uniform(0.5, 2, cfg.n_voxels).astype(np.float32))
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    whole = torch.empty(cfg.n_voxels, device="cuda")
    rec.error_image(dev(ev), f0, whole)
    for P in (2, 3, 8):
        acc = torch.zeros(cfg.n_voxels, device="cuda", dtype=torch.float64)
        for r in range(P):
            b, e = pkg.block_range(len(ev), r, P)
            part = torch.empty(cfg.n_voxels, device="cuda")
            rec.error_image(dev(ev[b:e]), f0, part)
            acc += part.double()
        torch.testing.assert_close(acc.float(), whole, rtol=1e-5, atol=1e-9)
    rec.close()


def test_timing_stats(pkg):
    cfg, ev, s = inputs("C1")
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.set_timing(True)
    rec.subset_step(dev(ev[:cfg.n_events]), f)
    st = rec.stats()
    assert st["timed_subsets"] == 1 and st["project_ms"] > 0 and st["update_ms"] > 0
    rec.close()


# ------------------------------------------------------------------ paper-shaped configs
@pytest.mark.parametrize("name", ["C2", "C5"])
def test_one_subset_paper_shaped(pkg, name):
    """One full 10^6-event subset (configs[1] / configs[4]) against the oracle."""
    cfg = lmgen.CONFIGS[name]
    ev = lmgen.subset_events(cfg, 0)
    s = lmgen.norm(cfg)
    f0 = np.ones(cfg.n_voxels)
    got = gpu_subset(pkg, cfg, ev, s, f0)
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev, s, f0)
    assert maxrel(got, ref) <= MAXREL_SUBSET


@pytest.mark.parametrize("name", ["C2", "C5"])
def test_full_reconstruction_paper_shaped(pkg, name):
    """configs[1] / configs[4]: 10 subsets x 10^6 events, 1 iteration, relative L2 after
    the reconstruction (and the per-voxel bar of one subset, compounded over 10)."""
    cfg, ev, s = inputs(name)
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.reconstruct(dev(ev), off, 1, f)
    rec.synchronize()
    got = f.cpu().numpy().astype(np.float64)
    rec.close()
    ref = oracle.reconstruct(oracle.geom(cfg.dims, cfg.voxel_mm), ev, off, 1, s, np.ones(cfg.n_voxels))
    assert rel_l2(got, ref) <= REL_L2_RECON
    assert maxrel(got, ref) <= 10 * MAXREL_SUBSET
    assert np.all(got > 0)


def test_c4_full_size_properties(pkg):
    """configs[3] at full size (300x300x560, 10^7 events in one subset): the oracle
    checks sampled forward projections one by one; the back-projection is checked by
    count conservation sum_{c>0} s f_new = N_eff, which holds at any size."""
    cfg = lmgen.CONFIGS["C4"]
    ev = lmgen.subset_events(cfg, 0)
    s = lmgen.norm(cfg)
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    assert rec.slabs > 1  # 200 MB images: the z-slab (out-of-L2) form runs
    f0 = np.ones(cfg.n_voxels, np.float32)
    evd = dev(ev)
    # sampled forward projections
    idx = np.random.default_rng(5).choice(len(ev), 2000, replace=False)
    fp = torch.empty(len(idx), device="cuda")
    rec.forward(dev(ev[idx]), dev(f0), fp)
    ref_fp = oracle.forward(g, ev[idx], f0)
    m = ref_fp > 0
    assert np.max(np.abs(fp.cpu().numpy()[m] - ref_fp[m]) / ref_fp[m]) <= 2e-6
    # count conservation of the full subset (every C4 LOR passes through its emission
    # point inside the phantom, so N_eff = N with f0 = 1)
    assert np.all(ref_fp > 0)
    f = dev(f0)
    c = torch.empty(cfg.n_voxels, device="cuda")
    rec.error_image(evd, f, c)
    cs = c.cpu().numpy().astype(np.float64)
    assert abs(cs.sum() - len(ev)) <= 1e-4 * len(ev)
    rec.update(f, c)
    rec.synchronize()
    got = f.cpu().numpy().astype(np.float64)
    hit = cs > 0
    total = float(np.sum(s.astype(np.float64)[hit] * got[hit]))
    assert abs(total - len(ev)) <= 1e-4 * len(ev)
    assert np.all(got > 0) and np.all(got[~hit] == 1.0)
    assert torch.count_nonzero(c).item() == 0  # the update re-zeroes c
    rec.close()


def test_c4_full_subset_matches_oracle(pkg):
    """configs[3] at full size, element by element: one 10^7-event subset through
    lmosem_subset_step in the launch configuration bench.py times (automatic z-slab
    count), against the oracle's subset step over the same events (~20 s of host work)."""
    cfg = lmgen.CONFIGS["C4"]
    ev = lmgen.subset_events(cfg, 1)
    s = lmgen.norm(cfg)
    f0 = np.random.default_rng(12).uniform(0.5, 2.0, cfg.n_voxels).astype(np.float32)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    assert rec.slabs > 1
    f = dev(f0)
    rec.subset_step(dev(ev), f)
    rec.synchronize()
    got = f.cpu().numpy().astype(np.float64)
    rec.close()
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev, s, f0)
    assert maxrel(got, ref) <= MAXREL_SUBSET


# ------------------------------------------------------------------ z-slab (out-of-L2) form
@pytest.mark.parametrize("slabs", [2, 3, 5])
def test_zslab_passes_match_oracle_c1(pkg, slabs):
    """The z-slab two-pass form of step 1 (pass A: per-slab partial forward projections,
    pass B: per-slab back-projection with the complete fp) gives the oracle's subset."""
    cfg, ev, s = inputs("C1")
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    rec.set_slabs(slabs)
    assert rec.slabs == slabs
    f0 = np.random.default_rng(11).uniform(0.5, 2.0, cfg.n_voxels)
    f = dev(f0.astype(np.float32))
    rec.subset_step(dev(ev[:cfg.n_events]), f)
    rec.synchronize()
    got = f.cpu().numpy().astype(np.float64)
    rec.close()
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev[:cfg.n_events], s, f0.astype(np.float32))
    assert maxrel(got, ref) <= MAXREL_SUBSET


def test_zslab_passes_match_oracle_c2(pkg):
    cfg = lmgen.CONFIGS["C2"]
    ev = lmgen.subset_events(cfg, 3)
    s = lmgen.norm(cfg)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    assert rec.slabs == 1  # 27 MB brick image: single fused pass
    rec.set_slabs(4)
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.subset_step(dev(ev), f)
    rec.synchronize()
    got = f.cpu().numpy().astype(np.float64)
    rec.close()
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev, s, np.ones(cfg.n_voxels))
    assert maxrel(got, ref) <= MAXREL_SUBSET


# ------------------------------------------------------------------ sensitivity image (NEXT-3)
@pytest.mark.parametrize("name,n,slabs", [("C1", 10_000, 0), ("C2", 100_000, 0), ("C2", 50_000, 3)])
def test_sensitivity_matches_oracle(pkg, name, n, slabs):
    cfg = lmgen.CONFIGS[name]
    ev = lmgen.events(cfg, 0, n)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(np.ones(cfg.n_voxels, np.float32)))
    rec.set_slabs(slabs)
    out = torch.empty(cfg.n_voxels, device="cuda")
    rec.sensitivity(dev(ev), out)
    rec.synchronize()
    got = out.cpu().numpy().astype(np.float64)
    rec.close()
    ref = oracle.sensitivity(oracle.geom(cfg.dims, cfg.voxel_mm), ev)
    assert np.all((got > 0) == (ref > 0))
    # s enters the update as a divisor: the one-subset bar of north_star applies
    assert maxrel(got, ref) <= MAXREL_SUBSET
    assert abs(got.sum() - ref.sum()) <= 1e-6 * ref.sum()


def test_set_norm_from_sensitivity(pkg):
    """A sensitivity computed on the GPU, installed with set_norm, drives the update."""
    cfg, ev, _ = inputs("C1")
    ev0 = ev[:cfg.n_events]
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, np.ones(cfg.n_voxels, np.float32))
    sens = torch.empty(cfg.n_voxels, device="cuda")
    rec.sensitivity(dev(ev0), sens)
    rec.set_norm(sens)
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.subset_step(dev(ev0), f)
    rec.synchronize()
    got = f.cpu().numpy().astype(np.float64)
    rec.close()
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    s_ref = oracle.sensitivity(g, ev0).astype(np.float32)
    ref = oracle.subset_step(g, ev0, s_ref, np.ones(cfg.n_voxels))
    assert maxrel(got, ref) <= MAXREL_SUBSET


def test_nccl_combine_single_rank(pkg):
    """The NCCL path (communicator from a broadcast id, in-place all-reduce of c on the
    compute stream) on the one GPU available: a 1-rank context must match the plain one."""
    cfg, ev, s = inputs("C1")
    ev0 = dev(ev[:cfg.n_events])
    rec0 = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    rec1 = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), dist=(0, 1, pkg.nccl_unique_id()))
    f0 = dev(np.ones(cfg.n_voxels, np.float32))
    f1 = dev(np.ones(cfg.n_voxels, np.float32))
    rec0.subset_step(ev0, f0)
    rec1.subset_step(ev0, f1)
    rec0.synchronize()
    rec1.synchronize()
    torch.testing.assert_close(f1, f0, rtol=1e-6, atol=0)
    rec0.close()
    rec1.close()


@pytest.mark.parametrize("combine", [1, 2, 3])
def test_combine_modes_single_rank(pkg, combine):
    """The combines on a 1-rank communicator — all-reduce + full update, the paper's
    PSD -> ISD switch (reduce-scatter, block update, all-gather),
    and the fused one-kernel ISD over NCCL symmetric windows (peer-pointer path) —
    through subset_step and a multi-subset reconstruct, against the oracle."""
    cfg, ev, s = inputs("C1")
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), dist=(0, 1, pkg.nccl_unique_id()))
    try:
        rec.set_combine(combine)
    except pkg.LmosemError as e:  # the fused mode needs NCCL symmetric windows + device comm
        rec.close()
        pytest.skip(f"combine {combine} unavailable: {e}")
    assert rec.combine == combine
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.subset_step(dev(ev[:cfg.n_events]), f)
    rec.synchronize()
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    ref = oracle.subset_step(g, ev[:cfg.n_events], s, np.ones(cfg.n_voxels))
    assert maxrel(f.cpu().numpy().astype(np.float64), ref) <= MAXREL_SUBSET
    f2 = dev(np.ones(cfg.n_voxels, np.float32))
    rec.reconstruct(dev(ev), off, 2, f2)
    rec.synchronize()
    ref2 = oracle.reconstruct(g, ev, off, 2, s, np.ones(cfg.n_voxels))
    assert rel_l2(f2.cpu().numpy().astype(np.float64), ref2) <= REL_L2_RECON
    rec.close()


@pytest.mark.parametrize("dims,vox", [((17, 12, 9), (1.0, 0.75, 1.5)), ((33, 5, 64), (0.6, 2.0, 0.45)),
                                      ((1, 40, 7), (1.0, 1.0, 1.0)),
                                      ((1170, 6, 5), (0.25, 1.0, 1.0)), ((3, 1170, 4), (1.0, 0.2, 1.0)), ((1210, 6, 5), (0.25, 1.0, 1.0)),
                                      ((1500, 8, 8), (0.2, 1.0, 1.0)), ((5, 3000, 4), (1.0, 0.1, 1.0)),
                                      ((6, 4, 2500), (1.0, 1.0, 0.15))])
def test_odd_extents_anisotropic_voxels(pkg, dims, vox):
    """Odd extents (padding, halo), anisotropic voxels (dominant axis in voxel units) and
    segments that start or end inside the volume, against the oracle. 1170 voxels is the
    longest clip box the path buffer holds (3 * 1170 pieces per warp and the clip area fill the 227 KB of
    shared memory, 1 CTA per SM); a longer axis (1500, 2500, 3000) is cut into slabs of at
    most 1170 voxels, each back-projected with the complete fp of its LORs."""
    g = oracle.geom(dims, vox)
    V = int(np.prod(dims))
    half = 0.5 * np.asarray(dims) * np.asarray(vox)
    rng = np.random.default_rng(sum(dims))
    n = 3000
    c = rng.uniform(-half, half, (n, 3))
    d = rng.normal(size=(n, 3))
    d /= np.linalg.norm(d, axis=1, keepdims=True)
    r = rng.uniform(0.2, 1.5, (n, 1)) * np.linalg.norm(half)  # some segments end inside
    ev = np.concatenate([c - r * d, c + r * d], axis=1).astype(np.float32)
    s = rng.uniform(0.5, 1.0, V).astype(np.float32)
    f0 = rng.uniform(0.5, 2.0, V)
    rec = pkg.Reconstructor(dims, vox, dev(s))
    fp = torch.empty(n, device="cuda")
    rec.forward(dev(ev), dev(f0.astype(np.float32)), fp)
    f = dev(f0.astype(np.float32))
    rec.subset_step(dev(ev), f)
    rec.synchronize()
    ref_fp = oracle.forward(g, ev, f0.astype(np.float32))
    m = ref_fp > 0
    assert np.all((fp.cpu().numpy() > 0) == m)
    # short segments (ending inside the volume): the slab-local crossings carry ~1e-7
    # voxel absolute error, so the per-event bar gets a 1e-6 f*mm floor
    err = np.abs(fp.cpu().numpy()[m] - ref_fp[m])
    assert np.all(err <= 2e-6 * ref_fp[m] + 1e-6), float(np.max(err / ref_fp[m]))
    ref = oracle.subset_step(g, ev, s, f0.astype(np.float32))
    assert maxrel(f.cpu().numpy().astype(np.float64), ref) <= MAXREL_SUBSET
    if max(dims) > 1170:  # slabs along the long axis, also for the sensitivity image
        assert rec.slabs >= 2
        sens = torch.empty(V, device="cuda")
        rec.sensitivity(dev(ev), sens)
        ref_s = oracle.sensitivity(g, ev)
        # s enters the update as a divisor: the one-subset bar (as test_sensitivity_matches_oracle)
        assert maxrel(sens.cpu().numpy().astype(np.float64), ref_s) <= MAXREL_SUBSET
    rec.close()


# ------------------------------------------------------------------ list-mode file streaming (NEXT-4)
def test_reconstruct_file_matches_device(pkg, tmp_path):
    """PAPER.md Listing 2 l.2-3 (read_events per subset): events streamed from a raw
    list-mode file (pread into pinned double buffers) give the device-resident result."""
    cfg, ev, s = inputs("C1")
    path = tmp_path / "c1.lm"
    ev.tofile(path)
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    fd = dev(np.ones(cfg.n_voxels, np.float32))
    rec.reconstruct(dev(ev), off, 2, fd)
    ff = dev(np.ones(cfg.n_voxels, np.float32))
    rec.reconstruct_file(str(path), off, 2, ff)
    rec.synchronize()
    torch.testing.assert_close(ff, fd, rtol=1e-5, atol=0)
    # errors: missing file, file shorter than the offsets -> EIO, context still usable
    with pytest.raises(pkg.LmosemError) as e:
        rec.reconstruct_file(str(tmp_path / "missing.lm"), off, 1, ff)
    assert e.value.status == 6
    short = tmp_path / "short.lm"
    ev[:cfg.n_events].tofile(short)
    with pytest.raises(pkg.LmosemError) as e:
        rec.reconstruct_file(str(short), off, 1, ff)
    assert e.value.status == 6
    rec.subset_step(dev(ev[:cfg.n_events]), ff)
    rec.synchronize()
    rec.close()


def test_user_stream_and_argument_errors(pkg):
    """Work enqueued on a non-default torch stream stays ordered with torch ops on it;
    bad offsets / iteration counts are EINVAL and leave the context usable."""
    cfg, ev, s = inputs("C1")
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    side = torch.cuda.Stream()
    with torch.cuda.stream(side):
        rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), stream=side)
        evd = torch.from_numpy(ev).cuda(non_blocking=False)
        f = torch.ones(cfg.n_voxels, device="cuda")
        rec.reconstruct(evd, off, 1, f)
        f2 = f * 1.0  # torch op on the same stream, after the library's work
    side.synchronize()
    ref = oracle.reconstruct(oracle.geom(cfg.dims, cfg.voxel_mm), ev, off, 1, s, np.ones(cfg.n_voxels))
    assert rel_l2(f2.cpu().numpy().astype(np.float64), ref) <= REL_L2_RECON
    for bad_off, iters in [(off[::-1].copy(), 1), (off - 5, 1), (off, -1)]:
        with pytest.raises((pkg.LmosemError, ValueError)):  # the binding checks offsets first
            rec.reconstruct(evd, bad_off, iters, f)
        o = np.ascontiguousarray(bad_off, np.int64)  # the C side's own check (EINVAL)
        assert rec._lib.lmosem_reconstruct(rec._h, evd.data_ptr(), o.ctypes.data, o.size - 1, iters,
                                           f.data_ptr()) == 1
    g0 = f.clone()
    rec.reconstruct(evd, off, 0, f)  # zero iterations: f unchanged
    rec.synchronize()
    assert torch.equal(f, g0)
    # pageable host memory passed as a device buffer through the raw C ABI: EINVAL before
    # anything is enqueued, the context stays usable; pinned host memory is accepted (UVA)
    lib, h = rec._lib, rec._h
    ev_host = np.ascontiguousarray(ev[:64])
    f_host = np.ones(cfg.n_voxels, np.float32)
    assert lib.lmosem_subset_step(h, ev_host.ctypes.data, 64, f.data_ptr()) == 1
    assert b"device-accessible" in lib.lmosem_last_error(h)
    assert lib.lmosem_subset_step(h, evd.data_ptr(), 64, f_host.ctypes.data) == 1
    assert lib.lmosem_update(h, f_host.ctypes.data, f.data_ptr()) == 1
    ev_pinned = torch.from_numpy(ev[:64].copy()).pin_memory()
    f3 = torch.ones(cfg.n_voxels, device="cuda")
    f4 = torch.ones(cfg.n_voxels, device="cuda")
    assert lib.lmosem_subset_step(h, ev_pinned.data_ptr(), 64, f3.data_ptr()) == 0
    rec.subset_step(evd[:64], f4)
    rec.synchronize()
    torch.testing.assert_close(f3, f4, rtol=1e-6, atol=0)
    rec.close()


def test_pathological_coordinates_do_not_fault(pkg):
    """Events with coordinates float64 cannot resolve against the volume (|p| ~ 1e20-1e38
    mm), near-coincident endpoints and subnormal separations must not fault the kernel or
    disturb the other events' result (they contribute nothing or a valid path)."""
    cfg, ev, s = inputs("C1")
    good = ev[:2000]
    big = np.float32(1e30)
    bad = np.array([[-big, 0.3, 0.2, big, 0.3, 0.2],
                    [-3e38, -3e38, -3e38, 3e38, 3e38, 3e38],
                    [1e20, 1e-20, 0.0, -1e20, 2e-20, 0.1],
                    [0.1, 0.2, 0.3, 0.1, 0.2, np.nextafter(np.float32(0.3), np.float32(1))],
                    [-7.0, 1e-30, 0.5, 7.0, -1e-30, 0.5]], np.float32)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.subset_step(dev(np.concatenate([good, bad])), f)
    rec.synchronize()  # would raise on an illegal address
    got = f.cpu().numpy().astype(np.float64)
    assert np.all(np.isfinite(got)) and np.all(got >= 0)
    rec.close()


@pytest.mark.parametrize("vox", [(0.3, 0.7, 1.1), (0.45, 1.3, 0.9), (1.0, 1.0, 1.0), (0.3, 0.9, 1.1)])
def test_lors_in_voxel_faces(pkg, vox):
    """Axis-parallel LORs lying exactly in voxel faces (float32 coordinates nearest to the
    planes lo + k*v, as crystal grids produce): the voxel row is a floating-point decision,
    taken by both sides as floor((p - lo) / v) in float64 (reading S6: the voxel above the
    face; a face that rounds to the upper outer face is outside)."""
    dims = (20, 16, 12)
    g = oracle.geom(dims, vox)
    lo = -0.5 * np.asarray(dims) * np.asarray(vox)
    rng = np.random.default_rng(7)
    ev = []
    for i in range(600):
        a = i % 3
        b, c = (a + 1) % 3, (a + 2) % 3
        p = np.zeros(3)
        # every face plane of axis b in turn (or the outer faces); (0.3, 0.9, 1.1): with 16
        # voxels of 0.9 mm the face k = 13 is one where floor((p - lo) * (1/v)) would be
        # one row lower than floor((p - lo) / v)
        p[b] = lo[b] + ((i // 3) % (dims[b] + 1)) * vox[b]
        p[c] = lo[c] + ((i // 7) % (dims[c] + 1)) * vox[c] if i % 2 else rng.uniform(lo[c], -lo[c])
        q = p.copy()
        p[a], q[a] = lo[a] - 3.0, -lo[a] + 3.0
        ev.append(np.concatenate([p, q]))
    ev = np.array(ev, np.float32)
    s = np.ones(int(np.prod(dims)), np.float32)
    f0 = rng.uniform(0.5, 2.0, int(np.prod(dims))).astype(np.float32)
    rec = pkg.Reconstructor(dims, vox, dev(s))
    fp = torch.empty(len(ev), device="cuda")
    rec.forward(dev(ev), dev(f0), fp)
    f = dev(f0)
    rec.subset_step(dev(ev), f)
    rec.synchronize()
    rec.close()
    ref_fp = oracle.forward(g, ev, f0)
    got_fp = fp.cpu().numpy().astype(np.float64)
    assert np.array_equal(got_fp > 0, ref_fp > 0)
    m = ref_fp > 0
    assert np.max(np.abs(got_fp[m] - ref_fp[m]) / ref_fp[m]) <= 2e-6
    ref = oracle.subset_step(g, ev, s, f0)
    assert maxrel(f.cpu().numpy().astype(np.float64), ref) <= MAXREL_SUBSET


def test_contexts_of_different_sizes_coexist(pkg):
    """Two contexts in one process, the small one created after the large one: each keeps
    working (the kernels' shared-memory limits are per function, process-wide) and their
    interleaved subsets give the same results as alone."""
    big, evb, sb = inputs("C1")
    cfg2 = lmgen.CONFIGS["C2"]
    ev2 = lmgen.subset_events(cfg2, 0, 20000)
    s2 = lmgen.norm(cfg2)
    rec_l = pkg.Reconstructor(cfg2.dims, cfg2.voxel_mm, dev(s2))
    rec_s = pkg.Reconstructor(big.dims, big.voxel_mm, dev(sb))
    fl = dev(np.ones(cfg2.n_voxels, np.float32))
    fs = dev(np.ones(big.n_voxels, np.float32))
    rec_l.subset_step(dev(ev2), fl)
    rec_s.subset_step(dev(evb[:big.n_events]), fs)
    rec_l.synchronize()
    rec_s.synchronize()
    ref_l = oracle.subset_step(oracle.geom(cfg2.dims, cfg2.voxel_mm), ev2, s2, np.ones(cfg2.n_voxels))
    ref_s = oracle.subset_step(oracle.geom(big.dims, big.voxel_mm), evb[:big.n_events], sb, np.ones(big.n_voxels))
    assert maxrel(fl.cpu().numpy().astype(np.float64), ref_l) <= MAXREL_SUBSET
    assert maxrel(fs.cpu().numpy().astype(np.float64), ref_s) <= MAXREL_SUBSET
    rec_l.close()
    rec_s.close()


def test_out_of_memory_is_enomem_and_recoverable(pkg):
    """A subset too large for the z-slab forward-projection array (4 B per event): ENOMEM,
    f untouched, the context keeps working; a context failure (ECUDA) makes every later
    call answer ESTATE (checked in a subprocess: a kernel fault poisons the CUDA context)."""
    cfg, ev, s = inputs("C1")
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    rec.set_slabs(2)
    evd = dev(ev[:cfg.n_events])
    f = dev(np.ones(cfg.n_voxels, np.float32))
    st = rec._lib.lmosem_subset_step(rec._h, evd.data_ptr(), 1 << 42, f.data_ptr())  # 16 TB fp array
    assert st == 2, rec._lib.lmosem_last_error(rec._h)
    rec.synchronize()
    assert torch.all(f == 1.0).item()
    rec.subset_step(evd, f)
    rec.synchronize()
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev[:cfg.n_events], s, np.ones(cfg.n_voxels))
    assert maxrel(f.cpu().numpy().astype(np.float64), ref) <= MAXREL_SUBSET
    rec.close()


ESTATE_SCRIPT = r"""
import ctypes, numpy as np, torch
import paper_conf_ipps_steuwerkg12_b200 as pkg
rec = pkg.Reconstructor((16, 16, 16), (1, 1, 1), torch.ones(4096, device="cuda"))
lib, h = rec._lib, rec._h
f = torch.ones(4096, device="cuda")
ev = torch.zeros(64, 6, device="cuda")
st1 = lib.lmosem_subset_step(h, ev.data_ptr(), 1 << 30, f.data_ptr())  # reads far past the buffer
st2 = lib.lmosem_synchronize(h)
st3 = lib.lmosem_subset_step(h, ev.data_ptr(), 64, f.data_ptr())
print(st1, st2, st3, lib.lmosem_last_error(h).decode()[:60])
print("destroy", lib.lmosem_destroy(h))
"""


def test_runtime_failure_poisons_context():
    """ECUDA (a kernel reading past the caller's event buffer) -> ESTATE afterwards."""
    import subprocess
    import sys
    if not torch.cuda.is_available():
        pytest.skip("needs a GPU")
    from conftest import ROOT
    out = subprocess.run([sys.executable, "-c", ESTATE_SCRIPT], capture_output=True, text=True, timeout=300,
                         cwd=ROOT)
    lines = out.stdout.strip().splitlines()
    assert lines, out.stderr[-2000:]
    st1, st2, st3 = (int(x) for x in lines[0].split()[:3])
    assert st1 == 0 and st2 == 3 and st3 == 5, lines
    assert lines[-1] == "destroy 0"


@pytest.mark.parametrize("slabs", [1, 3])
def test_programmatic_dependent_launch_on_off(pkg, monkeypatch, slabs):
    """The kernels of a reconstruction run as programmatic dependent launches (each waits,
    griddepcontrol.wait, before touching f, c or fp); LMOSEM_PDL=0 (read at lmosem_init)
    launches them plainly. Both orders reach the oracle's 3-subset result, and agree."""
    cfg = lmgen.CONFIGS["C2"]
    L, n = 3, 200_000
    ev = np.concatenate([lmgen.subset_events(cfg, l, n) for l in range(L)])
    s = lmgen.norm(cfg)
    off = np.arange(L + 1) * n
    f0 = np.random.default_rng(5).uniform(0.5, 2.0, cfg.n_voxels).astype(np.float32)
    got = {}
    for pdl in ("0", "1"):
        monkeypatch.setenv("LMOSEM_PDL", pdl)
        rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
        rec.set_slabs(slabs)
        f = dev(f0)
        rec.reconstruct(dev(ev), off, 1, f)
        rec.synchronize()
        got[pdl] = f.cpu().numpy().astype(np.float64)
        rec.close()
    ref = oracle.reconstruct(oracle.geom(cfg.dims, cfg.voxel_mm), ev, off, 1, s, f0.astype(np.float64))
    for pdl in ("0", "1"):
        assert maxrel(got[pdl], ref) <= 2 * MAXREL_SUBSET
        assert rel_l2(got[pdl], ref) <= REL_L2_RECON
    assert maxrel(got["1"], got["0"]) <= 1e-5


@pytest.mark.parametrize("slabs", [1, 3])
def test_zero_forward_projection_events_skipped(pkg, slabs):
    """Reading S7 (the division at PAPER.md line 464): an event whose forward projection is
    0 (its path only crosses voxels with f = 0) contributes nothing. f0 is zero outside a
    small ball, so most C1 events have fp = 0; the fused kernel and the z-slab passes must
    skip them (otherwise c = inf and f = 0 * inf = NaN on their paths)."""
    cfg, ev, s = inputs("C1")
    ev = ev[:cfg.n_events]
    nx, ny, nz = cfg.dims
    i = np.arange(cfg.n_voxels)
    ix, iy, iz = i % nx, (i // nx) % ny, i // (nx * ny)
    f0 = np.where((ix - 9) ** 2 + (iy - 7) ** 2 + (iz - 8) ** 2 <= 4, 1.5, 0.0).astype(np.float32)
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    fp = oracle.forward(g, ev, f0)
    assert (fp == 0).sum() > len(ev) // 2 and (fp > 0).sum() > 50  # both kinds present
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    rec.set_slabs(slabs)
    f = dev(f0)
    rec.subset_step(dev(ev), f)
    rec.synchronize()
    rec.close()
    got = f.cpu().numpy().astype(np.float64)
    ref = oracle.subset_step(g, ev, s, f0)
    assert np.all(np.isfinite(got))
    assert np.array_equal(got == 0, ref == 0)
    assert maxrel(got, ref) <= MAXREL_SUBSET


@pytest.mark.parametrize("wide_n", ["0", "1000000000"])
def test_fused_pass_cta_shapes(pkg, monkeypatch, wide_n):
    """The fused pass in both CTA shapes — MODE 6 (224 threads x 4 CTAs per SM, launches of
    >= LMOSEM_WIDE_N events) and MODE 5 (256 x 3) — on a C1 reconstruction and a 200k-event
    C2 subset against the oracle (LMOSEM_WIDE_N = 0: every launch MODE 6; 1e9: none)."""
    monkeypatch.setenv("LMOSEM_WIDE_N", wide_n)
    cfg, ev, s = inputs("C1")
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.reconstruct(dev(ev), off, 1, f)
    rec.synchronize()
    rec.close()
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    ref = oracle.reconstruct(g, ev, off, 1, s, np.ones(cfg.n_voxels))
    assert rel_l2(f.cpu().numpy().astype(np.float64), ref) <= REL_L2_RECON
    cfg2 = lmgen.CONFIGS["C2"]
    ev2 = lmgen.subset_events(cfg2, 3, 200_000)
    s2 = lmgen.norm(cfg2)
    got = gpu_subset(pkg, cfg2, ev2, s2, np.ones(cfg2.n_voxels))
    ref2 = oracle.subset_step(oracle.geom(cfg2.dims, cfg2.voxel_mm), ev2, s2, np.ones(cfg2.n_voxels))
    assert maxrel(got, ref2) <= MAXREL_SUBSET


@pytest.mark.parametrize("tex", ["0", "1"])
def test_lsu_and_texture_gathers(pkg, monkeypatch, tex):
    """The fused pass gathers f through the texture pipe (MODE 5) when the brick f fits a
    1-D linear texture, else (or with LMOSEM_TEX=0, read at lmosem_init) with LSU loads
    (MODE 0): both against the oracle on a C2-sized subset and through a reconstruction."""
    cfg = lmgen.CONFIGS["C2"]
    L, n = 2, 200_000
    ev = np.concatenate([lmgen.subset_events(cfg, l, n) for l in range(L)])
    s = lmgen.norm(cfg)
    off = np.arange(L + 1) * n
    f0 = np.random.default_rng(9).uniform(0.5, 2.0, cfg.n_voxels).astype(np.float32)
    monkeypatch.setenv("LMOSEM_TEX", tex)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    f = dev(f0)
    rec.reconstruct(dev(ev), off, 1, f)
    rec.synchronize()
    rec.close()
    got = f.cpu().numpy().astype(np.float64)
    ref = oracle.reconstruct(oracle.geom(cfg.dims, cfg.voxel_mm), ev, off, 1, s, f0.astype(np.float64))
    assert maxrel(got, ref) <= 2 * MAXREL_SUBSET
    assert rel_l2(got, ref) <= REL_L2_RECON


def test_misaligned_events_and_bad_offsets_rejected(pkg):
    """A device event array that is not 8-byte aligned is EINVAL before any launch (not a
    kernel fault), and the binding rejects subset offsets outside the events it was given;
    the context stays usable after both."""
    import ctypes
    cfg, ev, s = inputs("C1")
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    buf = dev(np.concatenate([[0.0], ev[:100].ravel()]).astype(np.float32))  # events at +4 B
    f = dev(np.ones(cfg.n_voxels, np.float32))
    lib = pkg.load()
    st = lib.lmosem_subset_step(rec._h, ctypes.c_void_p(buf.data_ptr() + 4), 100, ctypes.c_void_p(f.data_ptr()))
    assert st == 1  # EINVAL
    with pytest.raises(ValueError):
        rec.reconstruct(dev(ev[:100]), [0, 50, 101], 1, f)
    with pytest.raises(ValueError):
        rec.reconstruct_host(ev[:100], [0, 60, 40], 1, np.ones(cfg.n_voxels, np.float32))
    rec.subset_step(dev(ev[:cfg.n_events]), f)
    rec.synchronize()
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev[:cfg.n_events], s, np.ones(cfg.n_voxels))
    assert maxrel(f.cpu().numpy().astype(np.float64), ref) <= MAXREL_SUBSET
    rec.close()


def test_watchdog_aborts_stalled_combine(pkg, monkeypatch):
    """SURVEY.md §5 failure detection: a combine that does not finish (here a debug stall
    of 4 s in front of the NCCL collective, standing in for a dead peer) makes
    lmosem_synchronize return ENCCL within LMOSEM_TIMEOUT_S + 1 s instead of hanging; the
    context answers ESTATE, and lmosem_destroy aborts the communicator (the stall, like
    NCCL's kernels, polls the abort flag, so destroy returns promptly); the
    communicator is aborted and the context answers ESTATE afterwards."""
    import time
    monkeypatch.setenv("LMOSEM_TIMEOUT_S", "1")
    monkeypatch.setenv("LMOSEM_DEBUG_STALL_MS", "4000")
    cfg, ev, s = inputs("C1")
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), dist=(0, 1, pkg.nccl_unique_id()))
    f = dev(np.ones(cfg.n_voxels, np.float32))
    d_ev = dev(ev[:cfg.n_events])
    torch.cuda.synchronize()
    rec.subset_step(d_ev, f)
    t0 = time.time()
    with pytest.raises(pkg.LmosemError) as e:
        rec.synchronize()
    waited = time.time() - t0
    print(f"[watchdog] synchronize returned after {waited:.2f} s (timeout 1 s)")
    assert e.value.status in (3, 4) and waited < 2.0, (e.value, waited)  # ECUDA / ENCCL
    assert "LMOSEM_TIMEOUT_S" in str(e.value) or "nccl" in str(e.value)
    with pytest.raises(pkg.LmosemError) as e2:
        rec.subset_step(d_ev, f)
    assert e2.value.status == 5  # ESTATE
    t1 = time.time()
    rec.close()  # aborts the communicator; the stall exits on the abort flag
    print(f"[watchdog] destroy (ncclCommAbort) took {time.time() - t1:.2f} s")
    assert time.time() - t1 < 15.0  # NCCL's own abort (~1-2 s measured): it must not hang


def test_checkpoint_and_resume(pkg):
    """SURVEY.md §5 checkpoint / resume: the state between subsets is f alone (PAPER.md lines
    466-468). A C1 reconstruction of 2 iterations stopped after subset 0 of iteration 1 (f
    copied out = the checkpoint) and resumed with Reconstructor.resume in a NEW context
    equals the uninterrupted reconstruction and the oracle's."""
    cfg, ev, s = inputs("C1")
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    d_ev = dev(ev)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    f_full = dev(np.ones(cfg.n_voxels, np.float32))
    rec.reconstruct(d_ev, off, 2, f_full)
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.reconstruct(d_ev, off, 1, f)           # iteration 0
    rec.reconstruct(d_ev, off[:2], 1, f)       # iteration 1, subset 0 -> checkpoint
    rec.synchronize()
    ckpt = f.cpu().numpy().copy()
    rec.close()
    rec2 = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    f2 = dev(ckpt)
    rec2.resume(d_ev, off, 2, f2, start_iteration=1, start_subset=1)
    rec2.synchronize()
    rec2.close()
    got = f2.cpu().numpy().astype(np.float64)
    np.testing.assert_allclose(got, f_full.cpu().numpy().astype(np.float64), rtol=1e-5, atol=0)
    ref = oracle.reconstruct(oracle.geom(cfg.dims, cfg.voxel_mm), ev, off, 2, s, np.ones(cfg.n_voxels))
    assert rel_l2(got, ref) <= REL_L2_RECON
    with pytest.raises(ValueError):
        rec2 = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
        try:
            rec2.resume(d_ev, off, 2, f2, start_iteration=3, start_subset=0)
        finally:
            rec2.close()


def test_combine_autotune_at_init(pkg, monkeypatch):
    """The automatic P > 1 combine is chosen by timing (include/lmosem.h): after the fused
    combine's self-test, init times it, ISD and ALLREDUCE on this box and keeps the fastest. Forced here
    on a 1-rank communicator (LMOSEM_AUTO_FUSED=force): both times are reported, the choice
    is one of the two, and the result matches the oracle."""
    monkeypatch.setenv("LMOSEM_AUTO_FUSED", "force")
    cfg, ev, s = inputs("C1")
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s), dist=(0, 1, pkg.nccl_unique_id()))
    st = rec.stats()
    tf, ti, ta = st["tune_fused_ms"], st["tune_isd_ms"], st["tune_allreduce_ms"]
    print(f"[autotune] fused {tf:.4f} ms, isd {ti:.4f} ms, allreduce {ta:.4f} ms -> combine {rec.combine}")
    assert tf > 0 and ti > 0 and ta > 0
    assert rec.combine == (3 if tf <= ti and tf <= ta else (2 if ti <= ta else 1))
    f = dev(np.ones(cfg.n_voxels, np.float32))
    rec.subset_step(dev(ev[:cfg.n_events]), f)
    rec.synchronize()
    rec.close()
    ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev[:cfg.n_events], s, np.ones(cfg.n_voxels))
    assert maxrel(f.cpu().numpy().astype(np.float64), ref) <= MAXREL_SUBSET
