"""GPU parity of the listed z-slab form (DESIGN.md §7 "Listed z-slab form") against the
float64 oracle, through the C ABI.

k_zclass sorts a subset's events into per-launch lists: LORs inside one fine slab go to a
fused launch over that slab's box, the rest to passes A/B of the coarse slabs they meet.
Every split must give the oracle's subset (Listing 2) — in particular
for LORs lying in, ending on, or running along a slab plane, where the classification's
margin decides which launch owns them. LMOSEM_ZLIST=0 is the unlisted two-pass form,
1 coarse lists only, 2 (default) coarse + fine lists.
"""
import numpy as np
import pytest

import lmgen
import oracle

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

MAXREL_SUBSET = 1e-4


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


_ref = {}


def subset_case(name):
    if name not in _ref:
        cfg = lmgen.CONFIGS[name]
        n = cfg.n_events if name == "C1" else 300_000
        ev = lmgen.subset_events(cfg, 1, n)
        s = lmgen.norm(cfg)
        f0 = np.random.default_rng(5).uniform(0.5, 2.0, cfg.n_voxels).astype(np.float32)
        ref = oracle.subset_step(oracle.geom(cfg.dims, cfg.voxel_mm), ev, s, f0)
        _ref[name] = (cfg, ev, s, f0, ref)
    return _ref[name]


# (LMOSEM_ZLIST, ZFINE windows per coarse slab, ZFUSED_MODE, ZOVER window overlap, ZWIN width,
#  ZMERGE: the windows of a coarse slab in one launch, ZMED: medium-window stride divisor, 0 = none)
FORMS = [("0", "2", "6", "1", "0", "1", "3"), ("1", "2", "6", "1", "0", "1", "0"), ("1", "2", "6", "1", "0", "1", "3"),
         ("2", "2", "6", "1", "0", "1", "0"), ("2", "1", "6", "1", "0", "1", "3"), ("2", "3", "5", "1", "0", "1", "2"),
         ("2", "2", "6", "2", "0", "1", "3"), ("2", "3", "6", "3", "0", "1", "1"), ("2", "2", "5", "2", "0", "0", "3"),
         ("2", "2", "5", "2", "20", "1", "3"), ("2", "2", "5", "4", "8", "1", "3"), ("2", "2", "5", "4", "0", "1", "8")]


@pytest.mark.parametrize("zlist,zfine,zmode,zover,zwin,zmerge,zmed", FORMS)
@pytest.mark.parametrize("name,slabs", [("C1", 2), ("C1", 3), ("C1", 5), ("C2", 3)])
def test_listed_zslab_subset_matches_oracle(pkg, monkeypatch, zlist, zfine, zmode, zover, zwin, zmerge, zmed, name,
                                            slabs):
    """ZWIN=20 at C2 with 3 slabs: 27 windows, 9 centred in a coarse slab -> two merged launches
    (kMaxSeg = 8); ZWIN=8 at stride 2 would need > 32 lists at C2: the stride grows until they
    fit; ZMED=8 leaves no list budget for medium windows at C2 (none are made); C1 with 5
    slabs runs the unlisted form (listed needs <= 4 coarse slabs)."""
    for k, v in (("ZLIST", zlist), ("ZFINE", zfine), ("ZFUSED_MODE", zmode), ("ZOVER", zover), ("ZWIN", zwin),
                 ("ZMERGE", zmerge), ("ZMED", zmed)):
        monkeypatch.setenv("LMOSEM_" + k, v)
    cfg, ev, s, f0, ref = subset_case(name)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(s))
    rec.set_slabs(slabs)
    f = dev(f0)
    rec.subset_step(dev(ev), f)
    rec.synchronize()
    got = f.cpu().numpy().astype(np.float64)
    rec.close()
    assert maxrel(got, ref) <= MAXREL_SUBSET


def plane_events(dims, vox):
    """LORs in, on and along the slab planes of a 16^3 volume (C1 forced to 2 slabs: coarse
    planes z = 0, 8, 16 voxels; fine (2 per coarse) z = 0, 4, 8, 12, 16)."""
    nz = dims[2]
    lo = [-dims[k] * vox[k] / 2 for k in range(3)]
    z = lambda v: lo[2] + v * vox[2]  # noqa: E731
    x0, x1 = lo[0] - 3.0, lo[0] + dims[0] * vox[0] + 3.0
    out = []
    for zp in (0, 4, 8, 12, 16):
        for dz in (0.0, 1e-7, -1e-7, 2e-3, -2e-3, 0.5, -0.5):
            out.append([x0, 0.3, z(zp + dz), x1, -0.2, z(zp + dz)])          # along z = plane (+ offsets)
        out.append([x0, 0.1, z(zp), x1, 0.4, z(zp + 0.75)])                   # leaving a plane upwards
        out.append([x0, 0.1, z(zp), x1, 0.4, z(zp - 0.75)])                   # ... and downwards
        out.append([0.2, 0.1, z(zp - 1.0), 0.7, 0.3, z(zp)])                  # ending on a plane (inside)
        out.append([0.2, -2.1, z(zp), 0.7, 3.3, z(zp + 3.999)])               # inside one fine slab
        out.append([0.2, -2.1, z(zp + 1e-4), 0.7, 3.3, z(zp + 4.0 - 1e-4)])    # just inside (margin)
    for far in (40.0, 1e3, 1e5, 1e7):                                          # far endpoints (float32
        out.append([-far, 0.3, z(3.9), far, -0.2, z(4.2)])                    # classification falls
        out.append([-far, 0.3 * far, z(-0.5) - 1e-3 * far, far, -0.2, z(16.5) + 1e-3 * far])  # back)
    out.append([float("nan"), 0.0, 0.0, 1.0, 1.0, 1.0])                         # non-finite: dropped
    out.append([0.5, 0.5, z(6.0), 0.5, 0.5, z(6.0)])                          # zero length: dropped
    for k in range(40):                                                       # steep and z-dominant
        t = k / 40.0
        out.append([lo[0] + 3 + t, lo[1] + 5, z(-2.0), lo[0] + 9 - t, lo[1] + 11, z(nz + 2.0)])
        out.append([lo[0] + 2, lo[1] + 3 + t, z(3.5 + t), lo[0] + 14, lo[1] + 12, z(8.5 + 3 * t)])
    return np.array(out, np.float32)


@pytest.mark.parametrize("zlist,zover,zmerge,zmed", [("0", "1", "1", "3"), ("1", "1", "1", "0"), ("1", "1", "1", "3"),
                                                    ("2", "1", "1", "0"), ("2", "2", "1", "3"), ("2", "2", "0", "1"),
                                                    ("2", "4", "1", "3")])
def test_listed_zslab_plane_cases(pkg, monkeypatch, zlist, zover, zmerge, zmed):
    monkeypatch.setenv("LMOSEM_ZLIST", zlist)
    monkeypatch.setenv("LMOSEM_ZOVER", zover)
    monkeypatch.setenv("LMOSEM_ZMERGE", zmerge)
    monkeypatch.setenv("LMOSEM_ZMED", zmed)
    cfg = lmgen.CONFIGS["C1"]
    ev = plane_events(cfg.dims, cfg.voxel_mm)
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    f0 = np.random.default_rng(3).uniform(0.5, 2.0, cfg.n_voxels).astype(np.float32)
    ref = oracle.error_image(g, ev, f0)
    rec = pkg.Reconstructor(cfg.dims, cfg.voxel_mm, dev(np.ones(cfg.n_voxels, np.float32)))
    rec.set_slabs(2)
    c = torch.zeros(cfg.n_voxels, device="cuda")
    rec.error_image(dev(ev), dev(f0), c)
    rec.synchronize()
    got = c.cpu().numpy().astype(np.float64)
    rec.close()
    err = np.abs(got - ref)
    tol = 1e-4 * np.maximum(np.abs(ref), 1e-3 * np.abs(ref).max())
    print(f"[parity] plane cases: max abs err {err.max():.3e}, {len(ev)} LORs")
    assert np.all(err <= tol)
