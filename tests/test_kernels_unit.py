"""Unit tests of single kernels outside the full path (compiled from tests/cuda/*.cu with
nvcc against the package's kernel header): the ISD block update used after the
reduce-scatter and the fused ISD combine body with emulated ranks — multi-rank logic that
cannot run on one GPU through NCCL (it refuses two ranks on one device)."""
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


def test_combine_emu_compiles(tmp_path):
    assert os.access(build("combine_emu", str(tmp_path)), os.X_OK)


@pytest.mark.gpu
def test_fused_combine_emulated_ranks(tmp_path):
    """§8(f) NEXT-1: the fused ISD combine body with P = 1, 2, 3, 4, 8 emulated ranks on one
    GPU (each with its own c, brick f, norm; a global-memory team barrier): every rank ends
    with the same updated f — the rank-ordered sum of the c's, then f*c/s guarded — bitwise
    against the host, and with c re-zeroed; padding bricks untouched."""
    exe = build("combine_emu", str(tmp_path))
    res = subprocess.run([exe], capture_output=True, text=True, timeout=300)
    assert res.returncode == 0 and res.stdout.strip().endswith("ok"), res.stdout + res.stderr
