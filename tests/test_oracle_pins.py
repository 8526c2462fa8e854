"""Pins for the float64 oracle against what the paper and mathematics fix (no GPU).

The paper prints no LM-OSEM numbers, so the oracle is pinned by hand-derived
closed forms (tests/golden/), textbook identities, invariants and brute force; each test
names its pin (P1..P13, SURVEY.md §8(c) / DESIGN.md "Pins").
"""
import math

import numpy as np
import pytest

import lmgen
import oracle
from conftest import GOLDEN, read_golden_paths

G4 = oracle.geom((4, 4, 4), (1.0, 1.0, 1.0))


def _dict(coord, ln):
    d = {}
    for c, l in zip(coord.tolist(), ln.tolist()):
        assert c not in d, "a voxel appears twice on one path"
        d[c] = l
    return d


def _inside(dims, vox, pts):
    lo = -0.5 * np.asarray(dims) * np.asarray(vox)
    hi = -lo
    return np.all((pts >= lo) & (pts < hi), axis=-1)


def chord_by_bisection(dims, vox, p1, p2, k=20001):
    """|S ∩ box| without any slab/plane algebra: sample the segment densely, take the
    first and last inside samples, bisect the inside predicate to 1e-15 on both sides."""
    p1 = np.asarray(p1, float)
    p2 = np.asarray(p2, float)
    t = np.linspace(0.0, 1.0, k)
    ins = _inside(dims, vox, p1 + t[:, None] * (p2 - p1))
    if not ins.any():
        return 0.0
    i0, i1 = np.argmax(ins), k - 1 - np.argmax(ins[::-1])

    def bis(a_out, a_in):
        for _ in range(200):
            m = 0.5 * (a_out + a_in)
            if _inside(dims, vox, p1 + m * (p2 - p1)):
                a_in = m
            else:
                a_out = m
            if abs(a_in - a_out) < 1e-16:
                break
        return a_in

    a0 = t[i0] if i0 == 0 else bis(t[i0 - 1], t[i0])
    a1 = t[i1] if i1 == k - 1 else bis(t[i1 + 1], t[i1])
    return (a1 - a0) * float(np.linalg.norm(p2 - p1))


def random_lors(rng, dims, vox, n, margin=1.5):
    """Random segments with both endpoints outside a box slightly larger than the volume."""
    half = 0.5 * np.asarray(dims) * np.asarray(vox)
    out = []
    while len(out) < n:
        c = rng.uniform(-half, half)
        d = rng.normal(size=3)
        d /= np.linalg.norm(d)
        r = margin * np.linalg.norm(half) + 1.0
        out.append((c - r * d, c + r * d))
    return out


# ---------------------------------------------------------------- golden (hand-derived)
@pytest.mark.parametrize("case", read_golden_paths(), ids=lambda c: c[0])
def test_golden_paths(case):
    """Hand-derived closed-form paths (tests/golden/paths_4cube.txt): P3, P4, P5, S2, S6."""
    _, p1, p2, pairs = case
    coord, ln = oracle.siddon_path(G4, p1, p2)
    assert coord.tolist() == [c for c, _ in pairs]
    np.testing.assert_allclose(ln, [l for _, l in pairs], rtol=1e-13, atol=1e-14)
    # the brute-force box clip (the reference routine of P2/P10/P14) reaches the same
    # hand-derived path, face cases included (half-open voxel boxes, reading S6)
    bc, bl = oracle.boxclip_path(G4, p1, p2)
    got = dict(zip(bc.tolist(), bl.tolist()))
    assert sorted(got) == sorted(c for c, _ in pairs)
    np.testing.assert_allclose([got[c] for c, _ in pairs], [l for _, l in pairs], rtol=1e-13, atol=1e-14)


def test_golden_em_update():
    """Hand-derived one-subset update (tests/golden/em_4cube.txt), Listing 2 with s = 1."""
    cases = {c[0]: c for c in read_golden_paths()}
    ev = np.array([cases["G1"][1] + cases["G1"][2], cases["G2"][1] + cases["G2"][2]], np.float32)
    with open(f"{GOLDEN}/em_4cube.txt") as fh:
        line = [l for l in fh if l.strip() and not l.startswith("#")][0]
    expect = np.ones(64)
    for tok in line.split():
        j, v = tok.split(":")
        expect[int(j)] = float(v)
    f = oracle.subset_step(G4, ev, np.ones(64, np.float32), np.ones(64))
    np.testing.assert_allclose(f, expect, rtol=1e-14)
    assert abs(f[expect != 1].sum() - 2.0) < 1e-14


# ---------------------------------------------------------------- P1: chord sums
@pytest.mark.parametrize("dims,vox", [((4, 4, 4), (1, 1, 1)), ((7, 5, 9), (1.0, 2.0, 0.5)),
                                      ((16, 16, 16), (1, 1, 1)), ((150, 150, 280), (1, 1, 1))])
def test_p1_chord_sum(dims, vox):
    g = oracle.geom(dims, vox)
    rng = np.random.default_rng(11)
    for p1, p2 in random_lors(rng, dims, vox, 40):
        coord, ln = oracle.siddon_path(g, p1, p2)
        assert np.all(ln > 0)
        assert np.all((coord >= 0) & (coord < np.prod(dims)))
        ref = chord_by_bisection(dims, vox, p1, p2)
        assert abs(ln.sum() - ref) <= 1e-12 * max(1.0, ref)


# ---------------------------------------------------------------- P2: brute force
def test_p2_boxclip_vs_sampling():
    """The brute-force per-voxel clip is itself pinned by dense sampling along the chord:
    per-voxel length error of sampling <= 2 L / K."""
    dims, vox = (5, 4, 6), (1.0, 1.5, 0.8)
    g = oracle.geom(dims, vox)
    rng = np.random.default_rng(3)
    K = 200001
    lo = -0.5 * np.asarray(dims) * np.asarray(vox)
    for p1, p2 in random_lors(rng, dims, vox, 6):
        coord, ln = oracle.boxclip_path(g, p1, p2)
        L = float(np.linalg.norm(p2 - p1))
        t = (np.arange(K) + 0.5) / K
        pts = p1 + t[:, None] * (p2 - p1)
        ins = _inside(dims, vox, pts)
        idx = np.floor((pts[ins] - lo) / np.asarray(vox)).astype(int)
        j = idx[:, 0] + dims[0] * (idx[:, 1] + dims[1] * idx[:, 2])
        cnt = np.bincount(j, minlength=int(np.prod(dims))) * (L / K)
        full = np.zeros(int(np.prod(dims)))
        full[coord] = ln
        assert np.max(np.abs(full - cnt)) <= 2.0 * L / K + 1e-12


@pytest.mark.parametrize("dims,vox", [((4, 4, 4), (1, 1, 1)), ((8, 6, 10), (1.0, 1.0, 1.0)),
                                      ((16, 16, 16), (1, 1, 1)), ((9, 11, 7), (0.5, 1.25, 2.0))])
def test_p2_siddon_vs_boxclip(dims, vox):
    g = oracle.geom(dims, vox)
    rng = np.random.default_rng(5)
    for p1, p2 in random_lors(rng, dims, vox, 60):
        a = _dict(*oracle.siddon_path(g, p1, p2))
        b = _dict(*oracle.boxclip_path(g, p1, p2))
        assert set(a) == set(b)
        for j in a:
            assert abs(a[j] - b[j]) <= 1e-12 * max(1.0, b[j])


def test_p2_axis_parallel_and_segment_inside():
    """Axis-parallel and in-volume segments vs brute force (S2: a segment, not a line)."""
    dims, vox = (6, 5, 4), (1, 1, 1)
    g = oracle.geom(dims, vox)
    rng = np.random.default_rng(9)
    for _ in range(40):
        p1 = rng.uniform(-4, 4, 3)
        p2 = p1.copy()
        ax = rng.integers(0, 3, size=rng.integers(1, 3))
        p2[ax] += rng.uniform(-6, 6, len(ax))
        a = _dict(*oracle.siddon_path(g, p1, p2))
        b = _dict(*oracle.boxclip_path(g, p1, p2))
        assert set(a) == set(b)
        for j in a:
            assert abs(a[j] - b[j]) <= 1e-12


# ---------------------------------------------------------------- P3/P4 closed forms
@pytest.mark.parametrize("axis", [0, 1, 2])
def test_p3_axis_aligned(axis):
    """Axis-aligned LOR 0.37 voxel off the faces: n_axis voxels, each of length v_axis."""
    dims, vox = (6, 7, 9), (1.0, 2.0, 0.5)
    g = oracle.geom(dims, vox)
    lo = -0.5 * np.asarray(dims) * np.asarray(vox)
    idx = np.array([2, 3, 4])
    base = lo + (idx + 0.37) * np.asarray(vox)
    p1, p2 = base.copy(), base.copy()
    p1[axis] = lo[axis] - 5
    p2[axis] = -lo[axis] + 5
    coord, ln = oracle.siddon_path(g, p1, p2)
    n = dims[axis]
    exp = []
    for k in range(n):
        i = idx.copy()
        i[axis] = k
        exp.append(i[0] + dims[0] * (i[1] + dims[1] * i[2]))
    assert coord.tolist() == exp
    np.testing.assert_allclose(ln, vox[axis], rtol=1e-14)


@pytest.mark.parametrize("n", [2, 5, 16])
def test_p4_main_diagonal(n):
    """Main diagonal of an n^3 cube (corner ties): n voxels (i,i,i), each sqrt(3) d."""
    d = 0.75
    g = oracle.geom((n, n, n), (d, d, d))
    e = 0.5 * n * d + 1.0
    coord, ln = oracle.siddon_path(g, [-e] * 3, [e] * 3)
    assert coord.tolist() == [i * (1 + n + n * n) for i in range(n)]
    np.testing.assert_allclose(ln, math.sqrt(3) * d, rtol=1e-13)


# ---------------------------------------------------------------- P5 symmetry
def test_p5_swap_and_shift():
    dims, vox = (12, 10, 14), (1.0, 1.0, 1.0)
    g = oracle.geom(dims, vox)
    rng = np.random.default_rng(2)
    for _ in range(30):  # segments inside the grid before and after the shift
        p1 = rng.uniform([-2.5, -2, -3], [2.5, 2, 3])
        p2 = rng.uniform([-2.5, -2, -3], [2.5, 2, 3])
        c1, l1 = oracle.siddon_path(g, p1, p2)
        c2, l2 = oracle.siddon_path(g, p2, p1)
        assert c1.tolist() == c2[::-1].tolist()
        np.testing.assert_allclose(l1, l2[::-1], rtol=1e-12, atol=1e-13)
        # shift by whole voxels (2, -1, 3): the segment stays well inside the 12x10x14 grid
        s = np.array([2.0, -1.0, 3.0])
        c3, l3 = oracle.siddon_path(g, p1 + s, p2 + s)
        a, b = _dict(c1, l1), _dict(c3, l3)
        sh = 2 + dims[0] * (-1 + dims[1] * 3)
        big = {j + sh: l for j, l in a.items() if l > 1e-9}
        assert {j: l for j, l in b.items() if l > 1e-9}.keys() == big.keys()
        for j in big:
            assert abs(b[j] - big[j]) <= 1e-11


# ---------------------------------------------------------------- P6/P7 projection
def test_p6_constant_image_forward():
    cfg = lmgen.CONFIGS["C1"]
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    ev = lmgen.events(cfg, 0, 50)
    fp = oracle.forward(g, ev, np.full(cfg.n_voxels, 2.5))
    for i in range(50):
        ref = chord_by_bisection(cfg.dims, cfg.voxel_mm, ev[i, :3].astype(float), ev[i, 3:].astype(float))
        assert abs(fp[i] - 2.5 * ref) <= 1e-11 * max(1, ref)


def test_p7_single_event_update():
    """One event, s = 1, f = 1: f_new_j = a_ij / sum_j a_ij on the path, 1 elsewhere
    (a_ij from the brute-force clip, independent of the Siddon routine)."""
    dims, vox = (8, 8, 8), (1, 1, 1)
    g = oracle.geom(dims, vox)
    rng = np.random.default_rng(21)
    for p1, p2 in random_lors(rng, dims, vox, 5):
        ev = np.concatenate([p1, p2]).astype(np.float32)[None]
        coord, ln = oracle.boxclip_path(g, ev[0, :3], ev[0, 3:])
        f = oracle.subset_step(g, ev, np.ones(512, np.float32), np.ones(512))
        exp = np.ones(512)
        exp[coord] = ln / ln.sum()
        np.testing.assert_allclose(f, exp, rtol=1e-12)


# ---------------------------------------------------------------- P8/P9 invariants
@pytest.mark.parametrize("name", ["C1"])
def test_p8_count_conservation(name):
    cfg = lmgen.CONFIGS[name]
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    ev = lmgen.subset_events(cfg, 0)
    s = lmgen.norm(cfg)
    f0 = np.random.default_rng(0).uniform(0.5, 2.0, cfg.n_voxels)
    c = oracle.error_image(g, ev, f0)
    f1 = oracle.update(f0, c, s)
    n_eff = int(np.sum(oracle.forward(g, ev, f0) > 0))
    m = (c > 0) & (s > 0)
    assert n_eff > 0.9 * len(ev)
    assert abs(np.sum(s[m] * f1[m]) - n_eff) <= 1e-10 * n_eff


def test_p9_positivity():
    cfg = lmgen.CONFIGS["C1"]
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    ev = lmgen.events(cfg, 0, cfg.n_events * cfg.n_subsets)
    off = np.arange(cfg.n_subsets + 1) * cfg.n_events
    f = oracle.reconstruct(g, ev, off, 3, lmgen.norm(cfg), np.ones(cfg.n_voxels))
    assert np.all(f > 0) and np.all(np.isfinite(f))


# ---------------------------------------------------------------- P10 textbook EM
def test_p10_sparse_matrix_em():
    """Shepp-Vardi EM with A from the brute-force clip via scipy.sparse:
    f_new = f * (A^T (1 / A f)) / s (guarded), vs oracle.subset_step."""
    sp = pytest.importorskip("scipy.sparse")
    dims, vox = (6, 5, 7), (1.0, 1.2, 0.9)
    g = oracle.geom(dims, vox)
    V = int(np.prod(dims))
    rng = np.random.default_rng(4)
    lors = random_lors(rng, dims, vox, 80)
    ev = np.array([np.concatenate([a, b]) for a, b in lors], np.float32)
    rows, cols, vals = [], [], []
    for i in range(len(ev)):
        co, ln = oracle.boxclip_path(g, ev[i, :3], ev[i, 3:])
        rows += [i] * len(co)
        cols += co.tolist()
        vals += ln.tolist()
    A = sp.csr_matrix((vals, (rows, cols)), shape=(len(ev), V))
    f0 = rng.uniform(0.5, 1.5, V)
    s = rng.uniform(0.2, 1.0, V).astype(np.float32)
    s[::13] = 0.0  # guard: s <= 0 leaves f unchanged
    Af = A @ f0
    ratio = np.where(Af > 0, 1.0 / np.where(Af > 0, Af, 1), 0.0)
    c = A.T @ ratio
    exp = np.where((c > 0) & (s > 0), f0 * c / np.where(s > 0, s, 1), f0)
    got = oracle.subset_step(g, ev, s, f0)
    np.testing.assert_allclose(got, exp, rtol=1e-12)


# ---------------------------------------------------------------- P15 ordered subsets
def test_p15_ordered_subsets_em():
    """OSEM (Listing 2 line 1: the subsets in order, each an EM update from the
    previous one's image; lines 591-593: the pass over the subsets repeated): three unequal
    subsets x two iterations, each step the Shepp-Vardi update with that subset's A from the
    brute-force clip via scipy.sparse, vs oracle.reconstruct with the subsets' offsets."""
    sp = pytest.importorskip("scipy.sparse")
    dims, vox = (5, 6, 4), (1.1, 0.9, 1.0)
    g = oracle.geom(dims, vox)
    V = int(np.prod(dims))
    rng = np.random.default_rng(15)
    lors = random_lors(rng, dims, vox, 90)
    ev = np.array([np.concatenate([a, b]) for a, b in lors], np.float32)
    offsets = np.array([0, 20, 55, 90], np.int64)
    s = rng.uniform(0.3, 1.2, V).astype(np.float32)
    f0 = rng.uniform(0.5, 1.5, V)
    A_of = []
    for l in range(3):
        rows, cols, vals = [], [], []
        for r, i in enumerate(range(offsets[l], offsets[l + 1])):
            co, ln = oracle.boxclip_path(g, ev[i, :3], ev[i, 3:])
            rows += [r] * len(co)
            cols += co.tolist()
            vals += ln.tolist()
        A_of.append(sp.csr_matrix((vals, (rows, cols)), shape=(offsets[l + 1] - offsets[l], V)))
    exp = f0.copy()
    for _ in range(2):
        for A in A_of:
            Af = A @ exp
            c = A.T @ np.where(Af > 0, 1.0 / np.where(Af > 0, Af, 1), 0.0)
            exp = np.where((c > 0) & (s > 0), exp * c / s, exp)
    got = oracle.reconstruct(g, ev, offsets, 2, s, f0)
    np.testing.assert_allclose(got, exp, rtol=1e-11)


# ---------------------------------------------------------------- P11 EM monotonicity
def test_p11_likelihood_monotone():
    cfg = lmgen.CONFIGS["C1"]
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    ev = lmgen.events(cfg, 0, 3000)
    V = cfg.n_voxels
    s = np.zeros(V)
    for i in range(len(ev)):  # s_j = sum_i a_ij over the same events
        co, ln = oracle.siddon_path(g, ev[i, :3], ev[i, 3:])
        np.add.at(s, co, ln)
    s32 = s.astype(np.float32)
    f = np.ones(V)
    hit = s32 > 0

    def loglik(f):
        fp = oracle.forward(g, ev, f)
        return np.sum(np.log(fp[fp > 0])) - np.sum(s32[hit].astype(float) * f[hit])

    ll = [loglik(f)]
    for _ in range(6):
        f = oracle.subset_step(g, ev, s32, f)
        ll.append(loglik(f))
    assert all(b - a >= -1e-9 * abs(a) for a, b in zip(ll, ll[1:])), ll
    assert ll[-1] > ll[0]


# ---------------------------------------------------------------- P12 PSD split
@pytest.mark.parametrize("P", [2, 3, 8])
def test_p12_psd_split_invariance(P):
    """PAPER.md §IV.A (lines 476-485): step 1 over a block split of the events, summed,
    equals step 1 over the whole subset."""
    cfg = lmgen.CONFIGS["C1"]
    g = oracle.geom(cfg.dims, cfg.voxel_mm)
    ev = lmgen.subset_events(cfg, 1)
    f = np.random.default_rng(1).uniform(0.5, 2, cfg.n_voxels)
    whole = oracle.error_image(g, ev, f)
    n = len(ev)
    parts = sum(oracle.error_image(g, ev[(r * n) // P:((r + 1) * n) // P], f) for r in range(P))
    np.testing.assert_allclose(parts, whole, rtol=1e-12, atol=1e-15)


# ---------------------------------------------------------------- P13 Listing-2 literal
def test_p13_listing2_literal_update():
    """With s = 1 the update is Listing 2 line 17 exactly: if (c[j] > 0) f[j] *= c[j]."""
    rng = np.random.default_rng(8)
    f = rng.uniform(0.1, 3, 1000)
    c = rng.uniform(-1, 2, 1000)
    c[::7] = 0
    got = oracle.update(f, c, np.ones(1000, np.float32))
    exp = f.copy()
    for j in range(1000):
        if c[j] > 0.0:
            exp[j] *= c[j]
    assert np.array_equal(got, exp)


# ---------------------------------------------------------------- degenerate events
def test_degenerate_events_contribute_nothing():
    g = oracle.geom((8, 8, 8), (1, 1, 1))
    nan = float("nan")
    ev = np.array([[0, 0, 0, 0, 0, 0],            # p1 == p2
                   [10, 10, 10, 20, 20, 20],      # misses
                   [nan, 0, 0, 1, 1, 1],          # non-finite
                   [-9, 4, 0, 9, 4, 0]],          # in the upper outer face y = 4
                  np.float32)
    c = oracle.error_image(g, ev, np.ones(512))
    assert np.all(c == 0)


# ---------------------------------------------------------------- P14 sensitivity image
def test_p14_sensitivity_textbook_and_sum():
    """s = A^T 1 with A from the brute-force clip (scipy.sparse), and sum_j s_j equals the
    sum of the chords found by bisection."""
    sp = pytest.importorskip("scipy.sparse")
    dims, vox = (7, 6, 5), (1.0, 0.8, 1.3)
    g = oracle.geom(dims, vox)
    V = int(np.prod(dims))
    rng = np.random.default_rng(14)
    lors = random_lors(rng, dims, vox, 60)
    ev = np.array([np.concatenate([a, b]) for a, b in lors], np.float32)
    rows, cols, vals = [], [], []
    for i in range(len(ev)):
        co, ln = oracle.boxclip_path(g, ev[i, :3], ev[i, 3:])
        rows += [i] * len(co)
        cols += co.tolist()
        vals += ln.tolist()
    A = sp.csr_matrix((vals, (rows, cols)), shape=(len(ev), V))
    s = oracle.sensitivity(g, ev)
    np.testing.assert_allclose(s, A.T @ np.ones(len(ev)), rtol=1e-12, atol=1e-13)
    chords = sum(chord_by_bisection(dims, vox, ev[i, :3].astype(float), ev[i, 3:].astype(float))
                 for i in range(len(ev)))
    assert abs(s.sum() - chords) <= 1e-11 * chords
