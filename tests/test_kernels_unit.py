"""Unit tests of single kernels outside the full path (compiled from tests/cuda/*.cu with
nvcc against the package's kernel header): the ISD block update used after the
reduce-scatter, whose multi-rank form cannot run on one GPU through NCCL."""
import os
import subprocess

import pytest

from conftest import ROOT

CSRC = os.path.join(ROOT, "paper_conf_ipps_steuwerkg12_b200", "csrc")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")


def build(name, out_dir):
    exe = os.path.join(out_dir, name)
    cmd = [NVCC, "-gencode", "arch=compute_100a,code=sm_100a", "-O2", "-std=c++17", "-I", CSRC,
           os.path.join(ROOT, "tests", "cuda", name + ".cu"), "-o", exe]
    res = subprocess.run(cmd, capture_output=True, text=True)
    assert res.returncode == 0, res.stdout + res.stderr
    return exe


def test_k_update_block_compiles(tmp_path):
    assert os.access(build("k_update_block", str(tmp_path)), os.X_OK)


@pytest.mark.gpu
def test_k_update_block(tmp_path):
    """Block [b0, b1) updated and c re-zeroed; the rest of [0, zero_to) only re-zeroed;
    bitwise against the host (IEEE single division and product)."""
    exe = build("k_update_block", str(tmp_path))
    res = subprocess.run([exe], capture_output=True, text=True, timeout=120)
    assert res.returncode == 0 and res.stdout.strip().endswith("ok"), res.stdout + res.stderr
