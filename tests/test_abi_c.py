"""The C ABI from plain C: tests/c/abi_consumer.c (C99, the header + liblmosem.so + the CUDA
runtime, no Python or torch in the process) compiles and links here; on the GPU it runs
a C1 reconstruction through lmosem_reconstruct (device buffers) and
lmosem_reconstruct_host (host buffers), checked against the float64 oracle."""
import os
import subprocess

import numpy as np
import pytest

import lmgen
import oracle
from conftest import ROOT

PKG = os.path.join(ROOT, "paper_conf_ipps_steuwerkg12_b200")
CUDA = "/usr/local/cuda"


@pytest.fixture(scope="module")
def consumer(tmp_path_factory):
    from paper_conf_ipps_steuwerkg12_b200 import build as b
    b.build()
    exe = str(tmp_path_factory.mktemp("abi_c") / "abi_consumer")
    cmd = ["gcc", "-std=c99", "-Wall", "-Wextra", "-Werror", "-pedantic", "-O2",
           "-I", os.path.join(ROOT, "include"), "-isystem", os.path.join(CUDA, "include"),
           os.path.join(ROOT, "tests", "c", "abi_consumer.c"), "-o", exe,
           "-L", PKG, "-llmosem", f"-Wl,-rpath,{PKG}",
           "-L", os.path.join(CUDA, "lib64"), "-lcudart", f"-Wl,-rpath,{os.path.join(CUDA, 'lib64')}"]
    res = subprocess.run(cmd, capture_output=True, text=True)
    assert res.returncode == 0, res.stdout + res.stderr
    return exe


def test_c_consumer_compiles_and_links(consumer):
    """The header is clean C99 (-pedantic -Werror) and every call the consumer makes
    resolves against liblmosem.so at link time."""
    assert os.access(consumer, os.X_OK)
    out = subprocess.run(["nm", "-u", consumer], capture_output=True, text=True).stdout
    assert "lmosem_reconstruct_host" in out and "lmosem_init" in out


@pytest.mark.gpu
@pytest.mark.parametrize("iters", [1, 2])
def test_c_consumer_matches_oracle(consumer, tmp_path, iters):
    cfg = lmgen.CONFIGS["C1"]
    L = cfg.n_subsets
    ev = np.concatenate([lmgen.subset_events(cfg, l) for l in range(L)])
    s = lmgen.norm(cfg)
    ev.tofile(tmp_path / "ev.bin")
    s.tofile(tmp_path / "norm.bin")
    out = tmp_path / "f.bin"
    args = [consumer, *map(str, cfg.dims), *map(str, cfg.voxel_mm), str(tmp_path / "ev.bin"),
            str(tmp_path / "norm.bin"), str(len(ev)), str(L), str(iters), str(out)]
    res = subprocess.run(args, capture_output=True, text=True, timeout=300)
    assert res.returncode == 0, res.stdout + res.stderr
    assert res.stdout.strip().endswith("ok")
    got = np.fromfile(out, np.float32).astype(np.float64).reshape(2, -1)
    off = np.array([(len(ev) * l) // L for l in range(L + 1)], np.int64)
    ref = oracle.reconstruct(oracle.geom(cfg.dims, cfg.voxel_mm), ev, off, iters, s,
                             np.ones(cfg.n_voxels))
    m = ref > 1e-3 * ref.max()
    for g in got:  # device-buffer and host-buffer entry points
        assert float(np.linalg.norm(g - ref) / np.linalg.norm(ref)) <= 1e-3
        assert float(np.max(np.abs(g[m] - ref[m]) / ref[m])) <= 1e-4 * L * iters
