"""Seeded fuzz parity (GPU vs the float64 oracle, through the C ABI): random volume extents
and anisotropic voxel sizes, random LORs (directions over the sphere, segments that start,
end or lie entirely inside the volume, some axis-parallel, some missing the volume), random
f, norm and forced z-slab counts. Each case checks per-event forward projections and one
subset step against the oracle at the north_star tolerance."""
import os

import numpy as np
import pytest

import oracle

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

# LMOSEM_FUZZ_CASES / LMOSEM_FUZZ_SEED0 widen the sweep for long offline runs
# (profiles/r01_fuzz_long.txt); the default suite runs seeds 0..63
N_CASES = int(os.environ.get("LMOSEM_FUZZ_CASES", "64"))
SEED0 = int(os.environ.get("LMOSEM_FUZZ_SEED0", "0"))


@pytest.fixture(scope="module")
def pkg():
    if not torch.cuda.is_available():
        pytest.skip("needs a GPU")
    import paper_conf_ipps_steuwerkg12_b200 as p
    p.load()
    return p


def dev(a):
    return torch.from_numpy(np.ascontiguousarray(a)).cuda()


def case(seed):
    rng = np.random.default_rng(1000 + seed)
    dims = [int(x) for x in rng.integers(1, 48, 3)]
    if seed % 4 == 3:  # one long axis (odd and even path-buffer sizes, many slabs)
        dims[seed % 3] = int(rng.integers(100, 320))
    dims = tuple(dims)
    vox = tuple(float(x) for x in rng.uniform(0.3, 2.5, 3))
    half = 0.5 * np.asarray(dims) * np.asarray(vox)
    n = int(rng.integers(1, 4000))
    c = rng.uniform(-1.3 * half, 1.3 * half, (n, 3))  # some centres outside: misses
    d = rng.normal(size=(n, 3))
    zero = rng.random((n, 3)) < 0.08  # axis-parallel components
    d[zero] = 0.0
    d[np.all(d == 0, axis=1), 0] = 1.0
    d /= np.linalg.norm(d, axis=1, keepdims=True)
    r = rng.uniform(0.05, 2.0, (n, 1)) * np.linalg.norm(half)
    ev = np.concatenate([c - r * d, c + r * d], axis=1).astype(np.float32)
    V = int(np.prod(dims))
    s = rng.uniform(0.2, 1.0, V).astype(np.float32)
    s[rng.random(V) < 0.03] = 0.0  # reading S9: s = 0 leaves f unchanged
    f0 = rng.uniform(0.3, 3.0, V).astype(np.float32)
    slabs = int(rng.integers(0, 5))
    return dims, vox, ev, s, f0, slabs


@pytest.mark.parametrize("seed", range(SEED0, SEED0 + N_CASES))
def test_fuzz_matches_oracle(pkg, seed):
    dims, vox, ev, s, f0, slabs = case(seed)
    g = oracle.geom(dims, vox)
    rec = pkg.Reconstructor(dims, vox, dev(s))
    rec.set_slabs(slabs)
    fp = torch.empty(len(ev), device="cuda")
    rec.forward(dev(ev), dev(f0), fp)
    f = dev(f0)
    rec.subset_step(dev(ev), f)
    rec.synchronize()
    got_fp = fp.cpu().numpy().astype(np.float64)
    got = f.cpu().numpy().astype(np.float64)
    rec.close()
    ref_fp = oracle.forward(g, ev, f0)
    m = ref_fp > 0
    assert np.array_equal(got_fp > 0, m)
    # slab-local crossings carry ~1e-7 voxel absolute error: a 1e-6 (f * mm) floor
    err = np.abs(got_fp[m] - ref_fp[m])
    assert np.all(err <= 2e-6 * ref_fp[m] + 1e-6 * max(vox)), float(np.max(err / ref_fp[m]))
    ref = oracle.subset_step(g, ev, s, f0)
    mm = ref > 1e-3 * ref.max()
    rel = np.abs(got[mm] - ref[mm]) / ref[mm]
    assert float(rel.max()) <= 1e-4, (dims, vox, slabs, float(rel.max()))
    assert np.array_equal(got[s == 0], f0.astype(np.float64)[s == 0])


@pytest.mark.parametrize("seed", range(SEED0, SEED0 + max(1, (12 * N_CASES) // 64)))
def test_fuzz_reconstruct_paths(pkg, seed, tmp_path):
    """Random subset offsets (empty subsets included) and iteration counts through the
    device, host and file entry points against the oracle's reconstruction; sensitivity
    image of the same LORs against the oracle's."""
    dims, vox, ev, s, f0, slabs = case(100 + seed)
    rng = np.random.default_rng(seed)
    L = int(rng.integers(1, 6))
    cuts = np.sort(rng.integers(0, len(ev) + 1, L - 1))
    off = np.concatenate([[0], cuts, [len(ev)]]).astype(np.int64)
    iters = int(rng.integers(1, 3))
    g = oracle.geom(dims, vox)
    ref = oracle.reconstruct(g, ev, off, iters, s, f0.astype(np.float64))
    rec = pkg.Reconstructor(dims, vox, dev(s))
    rec.set_slabs(slabs)
    fd = dev(f0)
    rec.reconstruct(dev(ev), off, iters, fd)
    fh = f0.copy()
    rec.reconstruct_host(torch.from_numpy(ev).pin_memory(), off, iters, fh)
    path = tmp_path / "ev.lm"
    ev.tofile(path)
    ff = dev(f0)
    rec.reconstruct_file(str(path), off, iters, ff)
    sens = torch.empty(int(np.prod(dims)), device="cuda")
    rec.sensitivity(dev(ev), sens)
    rec.synchronize()
    rec.close()
    for got in (fd.cpu().numpy(), fh, ff.cpu().numpy()):
        got = got.astype(np.float64)
        assert float(np.linalg.norm(got - ref) / np.linalg.norm(ref)) <= 1e-3
        mm = ref > 1e-3 * ref.max()
        assert float(np.max(np.abs(got[mm] - ref[mm]) / ref[mm])) <= 1e-4 * (1 + L * iters)
    ref_s = oracle.sensitivity(g, ev)
    got_s = sens.cpu().numpy().astype(np.float64)
    ms = ref_s > 1e-3 * ref_s.max()
    assert float(np.max(np.abs(got_s[ms] - ref_s[ms]) / ref_s[ms])) <= 1e-4


@pytest.mark.parametrize("scale", [1e-3, 1e3])
@pytest.mark.parametrize("seed", range(4))
def test_fuzz_scaled_and_short(pkg, seed, scale):
    """The same geometry in other units (voxel sizes 1e-3 and 1e3 times larger) and very
    short segments (1e-3 to 1 voxel, both endpoints inside, often inside one voxel)."""
    dims, vox, ev, s, f0, slabs = case(200 + seed)
    rng = np.random.default_rng(300 + seed)
    vox = tuple(v * scale for v in vox)
    ev = ev.astype(np.float64) * scale
    half = 0.5 * np.asarray(dims) * np.asarray(vox)
    k = len(ev) // 3  # a third of the LORs replaced by short interior segments
    c = rng.uniform(-0.95 * half, 0.95 * half, (k, 3))
    d = rng.normal(size=(k, 3))
    d /= np.linalg.norm(d, axis=1, keepdims=True)
    ln = rng.uniform(1e-3, 1.0, (k, 1)) * min(vox)
    ev[:k] = np.concatenate([c - 0.5 * ln * d, c + 0.5 * ln * d], axis=1)
    ev = ev.astype(np.float32)
    g = oracle.geom(dims, vox)
    rec = pkg.Reconstructor(dims, vox, dev(s))
    rec.set_slabs(slabs)
    fp = torch.empty(len(ev), device="cuda")
    rec.forward(dev(ev), dev(f0), fp)
    f = dev(f0)
    rec.subset_step(dev(ev), f)
    rec.synchronize()
    rec.close()
    ref_fp = oracle.forward(g, ev, f0)
    got_fp = fp.cpu().numpy().astype(np.float64)
    m = ref_fp > 0
    assert np.array_equal(got_fp > 0, m)
    err = np.abs(got_fp[m] - ref_fp[m])
    assert np.all(err <= 2e-6 * ref_fp[m] + 1e-6 * max(vox)), float(np.max(err / ref_fp[m]))
    ref = oracle.subset_step(g, ev, s, f0)
    got = f.cpu().numpy().astype(np.float64)
    mm = ref > 1e-3 * ref.max()
    assert float(np.max(np.abs(got[mm] - ref[mm]) / ref[mm])) <= 1e-4


@pytest.mark.parametrize("seed", range(SEED0, SEED0 + max(1, (16 * N_CASES) // 64)))
def test_fuzz_loopback_world(pkg, seed):
    """Random emulated worlds (P = 1..8 ranks of the loopback transport on this GPU, one host
    thread each), random combine (ALLREDUCE / ISD / FUSED), random volume, voxel sizes,
    slab count and subset offsets (empty subsets included): a reconstruction through
    lmosem_reconstruct on every rank against the oracle's, with bitwise-equal replicas
    (PAPER.md lines 476-485, 509-518)."""
    import threading
    dims, vox, ev, s, f0, slabs = case(400 + seed)
    rng = np.random.default_rng(500 + seed)
    P = int(rng.integers(1, 9))
    combine = int(rng.integers(1, 4))
    L = int(rng.integers(1, 5))
    off = np.concatenate([[0], np.sort(rng.integers(0, len(ev) + 1, L - 1)), [len(ev)]]).astype(np.int64)
    g = oracle.geom(dims, vox)
    ref = oracle.reconstruct(g, ev, off, 1, s, f0.astype(np.float64))
    group = pkg.Loopback(P)
    recs = [pkg.Reconstructor(dims, vox, dev(s), stream=torch.cuda.Stream(), loopback=(group, r)) for r in range(P)]
    fs = []
    for rec in recs:
        rec.set_slabs(slabs)
        rec.set_combine(combine)
        fs.append(dev(f0))
    d_ev = dev(ev)
    torch.cuda.synchronize()
    errs = []

    def work(r):
        try:
            recs[r].reconstruct(d_ev, off, 1, fs[r])
            recs[r].synchronize()
        except Exception as e:  # noqa: BLE001
            errs.append(e)
    th = [threading.Thread(target=work, args=(r,)) for r in range(P)]
    for t in th:
        t.start()
    for t in th:
        t.join(timeout=300)
    assert not errs, errs
    out = [f.cpu().numpy() for f in fs]
    for rec in recs:
        rec.close()
    group.close()
    for r in range(1, P):
        assert np.array_equal(out[r], out[0]), (P, combine, r)
    got = out[0].astype(np.float64)
    assert float(np.linalg.norm(got - ref) / np.linalg.norm(ref)) <= 1e-3, (P, combine, dims, slabs)
    mm = ref > 1e-3 * ref.max()
    assert float(np.max(np.abs(got[mm] - ref[mm]) / ref[mm])) <= 1e-4 * (1 + L), (P, combine, dims, slabs)
