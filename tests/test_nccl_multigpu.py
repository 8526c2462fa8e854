"""The real NCCL path at P > 1 (one process per GPU, tests/mp/nccl_parity_worker.py under
torchrun): every combine, including the fused multimem kernel and its init self-test, against
the float64 oracle with bitwise-equal replicas. Needs >= 2 visible GPUs; skipped on a
one-GPU box (where tests/test_loopback_gpu.py covers the same combine code with emulated
ranks)."""
import json
import os
import subprocess
import sys

import pytest

from conftest import ROOT

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu


def test_nccl_combines_across_gpus():
    if not torch.cuda.is_available() or torch.cuda.device_count() < 2:
        pytest.skip("needs >= 2 GPUs (NCCL refuses two ranks on one GPU)")
    g = min(8, torch.cuda.device_count())
    out = subprocess.run([sys.executable, "-m", "torch.distributed.run", "--nnodes", "1", "--nproc-per-node", str(g),
                          "--master-addr", "127.0.0.1", "--master-port", "29533",
                          os.path.join(ROOT, "tests", "mp", "nccl_parity_worker.py")],
                         capture_output=True, text=True, timeout=1200, cwd=ROOT)
    assert out.returncode == 0, out.stderr[-3000:]
    res = json.loads([ln for ln in out.stdout.splitlines() if ln.startswith("{")][-1])
    assert res["world"] == g
    for key, r in res.items():
        if key == "world" or "unavailable" in r:
            continue
        assert r["replicas_equal"], key
        bar = 1e-4 if "subset" in key else 10e-4
        assert r["max_rel"] <= bar and r["rel_l2"] <= 1e-3, (key, r)
    # the explicit modes 1 and 2 need no set-up: they must have run
    assert "unavailable" not in res["C2_subset_mode2"] and "unavailable" not in res["C2_subset_mode1"]
