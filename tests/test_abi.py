"""C-ABI boundary checks that need no GPU: the library loads, exports every symbol
include/lmosem.h declares, and validates arguments before touching CUDA."""
import ctypes
import os
import re

import numpy as np
import pytest

import paper_conf_ipps_steuwerkg12_b200 as pkg
from paper_conf_ipps_steuwerkg12_b200 import lmosem as L
from conftest import ROOT


@pytest.fixture(scope="module")
def lib():
    from paper_conf_ipps_steuwerkg12_b200 import build as b
    b.build()
    return pkg.load()


def header_functions():
    txt = open(os.path.join(ROOT, "include", "lmosem.h")).read()
    txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
    return sorted(set(re.findall(r"\b(lmosem_\w+)\s*\(", txt)))


def test_exports_every_declared_symbol(lib):
    decl = header_functions()
    assert len(decl) >= 15
    assert sorted(L.EXPORTS) == decl
    for name in decl:
        assert hasattr(lib, name), name
    out = os.popen(f"nm -D --defined-only {L.SO_PATH}").read()
    exported = set(re.findall(r"\bT (lmosem_\w+)", out))
    assert exported == set(decl), exported ^ set(decl)


def test_version(lib):
    assert pkg.version().startswith("lmosem") and "sm_100a" in pkg.version()


def test_block_range_partition(lib):
    for n in [0, 1, 7, 10_000, 1_000_000, 10_000_001]:
        for P in [1, 2, 3, 4, 8]:
            ranges = [pkg.block_range(n, r, P) for r in range(P)]
            assert ranges[0][0] == 0 and ranges[-1][1] == n
            for (b0, e0), (b1, _) in zip(ranges, ranges[1:]):
                assert e0 == b1
            for r, (b, e) in enumerate(ranges):
                assert b == (r * n) // P and e == ((r + 1) * n) // P
    big = 2**40
    assert pkg.block_range(big, 7, 8) == ((7 * big) // 8, big)


def test_isd_block_partition(lib):
    """The ISD combine's brick blocks (the NCCL reduce-scatter / all-gather chunks and the
    block update at P > 1): equal chunks of the padded allocation, rank order, real-brick
    parts partitioning [0, n_bricks)."""
    import paper_conf_ipps_steuwerkg12_b200 as pkg
    for nb in (0, 1, 7, 8, 1000, 27 * 10**5 + 13, 6735344):
        for P in (1, 2, 3, 4, 7, 8):
            blocks = [pkg.isd_block(nb, r, P) for r in range(P)]
            alloc = blocks[0][2]
            assert all(b[2] == alloc for b in blocks)
            assert alloc % P == 0 and nb <= alloc < nb + P
            chunk = alloc // P
            for r, (b, e, _) in enumerate(blocks):
                assert b == min(nb, r * chunk) and e == min(nb, (r + 1) * chunk)
            assert blocks[0][0] == 0 and blocks[-1][1] == nb
            assert all(blocks[r][1] == blocks[r + 1][0] for r in range(P - 1))
    for bad in ((-1, 0, 1), (10, 1, 1), (10, -1, 2), (10, 0, 0)):
        with pytest.raises(pkg.LmosemError):
            pkg.isd_block(*bad)


@pytest.mark.parametrize("args", [(-1, 0, 1), (10, -1, 2), (10, 2, 2), (10, 0, 0)])
def test_block_range_einval(lib, args):
    with pytest.raises(pkg.LmosemError) as e:
        pkg.block_range(*args)
    assert e.value.status == L.EINVAL


def _init(lib, dims, vox, norm_ptr=1, dist=None):
    h = ctypes.c_void_p(123)
    d = (ctypes.c_int32 * 3)(*dims)
    v = (ctypes.c_double * 3)(*vox)
    st = lib.lmosem_init(ctypes.byref(h), d, v, norm_ptr, dist)
    return st, h


@pytest.mark.parametrize("dims,vox", [((0, 4, 4), (1, 1, 1)), ((4, -1, 4), (1, 1, 1)),
                                      ((4, 4, 4), (0, 1, 1)), ((4, 4, 4), (1, float("nan"), 1)),
                                      ((4, 4, 4), (1, 1, float("inf"))), ((2048, 2048, 1024), (1, 1, 1)),
                                      ((4, 1211, 1211), (1, 1, 1)), ((1300, 2, 1300), (1, 1, 1))])
def test_init_einval_before_cuda(lib, dims, vox):
    st, h = _init(lib, dims, vox)
    assert st == L.EINVAL and not h.value


def test_init_einval_pointers_and_dist(lib):
    h = ctypes.c_void_p()
    d = (ctypes.c_int32 * 3)(4, 4, 4)
    v = (ctypes.c_double * 3)(1, 1, 1)
    assert lib.lmosem_init(None, d, v, 1, None) == L.EINVAL
    assert lib.lmosem_init(ctypes.byref(h), None, v, 1, None) == L.EINVAL
    assert lib.lmosem_init(ctypes.byref(h), d, v, None, None) == L.EINVAL
    for rank, world, uid in [(0, 0, 1), (2, 2, 1), (-1, 2, 1), (0, 2, None), (0, 1, None)]:
        dist = L.Dist(rank, world, uid)
        assert lib.lmosem_init(ctypes.byref(h), d, v, 1, ctypes.byref(dist)) == L.EINVAL


def test_null_context_calls(lib):
    assert lib.lmosem_destroy(None) == L.OK
    assert lib.lmosem_subset_step(None, None, 0, None) == L.EINVAL
    assert lib.lmosem_synchronize(None) == L.EINVAL
    assert isinstance(lib.lmosem_last_error(None), bytes)


def test_event_record_layout():
    """lmosem_event is 6 packed float32 (24 B), matching the generator's (n, 6) arrays."""
    import lmgen
    ev = lmgen.events(lmgen.CONFIGS["C1"], 0, 4)
    assert ev.dtype == np.float32 and ev.shape == (4, 6) and ev.strides == (24, 4)


def test_no_cpu_fallback_without_gpu(lib):
    torch = pytest.importorskip("torch")
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    with pytest.raises(RuntimeError):
        pkg.Reconstructor((4, 4, 4), (1, 1, 1), np.ones(64, np.float32))


def test_product_does_not_import_oracle():
    """The product package never references the oracle (independence)."""
    pdir = os.path.join(ROOT, "paper_conf_ipps_steuwerkg12_b200")
    for dp, _, files in os.walk(pdir):
        for fn in files:
            if fn.endswith((".py", ".cu", ".cuh", ".h", ".cpp")):
                txt = open(os.path.join(dp, fn)).read()
                assert not re.search(r"^\s*(import|from)\s+oracle\b|liboracle|oracle\.h|oracle_\w+\(", txt, re.M), fn


def test_l2peak_exports_and_rejects_bad_arguments(lib):
    """include/l2peak.h (the roofline microbenchmarks): libl2peak.so exports l2peak_run
    and rejects bad arguments with -1 before touching CUDA."""
    txt = re.sub(r"/\*.*?\*/", "", open(os.path.join(ROOT, "include", "l2peak.h")).read(), flags=re.S)
    decl = sorted(set(re.findall(r"\b(l2peak_\w+)\s*\(", txt)))
    so = os.path.join(os.path.dirname(L.SO_PATH), "libl2peak.so")
    out = os.popen(f"nm -D --defined-only {so}").read()
    assert set(re.findall(r"\bT (l2peak_\w+)", out)) == set(decl) == {"l2peak_run"}
    l2 = ctypes.CDLL(so)
    l2.l2peak_run.argtypes = [ctypes.c_int, ctypes.c_int64, ctypes.c_int32, ctypes.POINTER(ctypes.c_float),
                              ctypes.POINTER(ctypes.c_double)]
    ms, ops = ctypes.c_float(), ctypes.c_double()
    for mode, n, k in [(9, 1 << 20, 4), (-1, 1 << 20, 4), (0, 10, 4), (0, 1 << 20, 0), (0, 1 << 33, 4)]:
        assert l2.l2peak_run(mode, n, k, ctypes.byref(ms), ctypes.byref(ops)) == -1


def test_loopback_group_arguments(lib):
    """The loopback group (include/lmosem.h "Emulated world"): world 1..16, NULL checks and
    rank range before any CUDA call; destroy of an empty group and of NULL is OK."""
    h = ctypes.c_void_p()
    for bad in (0, -1, 17):
        assert lib.lmosem_loopback_create(bad, ctypes.byref(h)) == L.EINVAL and not h.value
    assert lib.lmosem_loopback_create(2, None) == L.EINVAL
    assert lib.lmosem_loopback_create(2, ctypes.byref(h)) == L.OK and h.value
    c = ctypes.c_void_p(123)
    d = (ctypes.c_int32 * 3)(4, 4, 4)
    v = (ctypes.c_double * 3)(1, 1, 1)
    for rank in (-1, 2):
        assert lib.lmosem_init_loopback(ctypes.byref(c), d, v, 1, h, rank) == L.EINVAL and not c.value
    assert lib.lmosem_init_loopback(ctypes.byref(c), d, v, 1, None, 0) == L.EINVAL
    assert lib.lmosem_loopback_destroy(h) == L.OK
    assert lib.lmosem_loopback_destroy(None) == L.OK
