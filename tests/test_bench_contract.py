"""bench.py's JSON-line contract: the reference (oracle) arm on CPU, and the CUDA arm on a
small config on the GPU (keys and types the driver and DESIGN.md §9 rely on)."""
import json
import os
import subprocess
import sys

import pytest

from conftest import ROOT

BENCH = os.path.join(ROOT, "bench.py")


def run_bench(args, env=None, timeout=600):
    e = dict(os.environ)
    e.update(env or {})
    out = subprocess.run([sys.executable, BENCH] + args, capture_output=True, text=True, timeout=timeout, cwd=ROOT,
                         env=e)
    assert out.returncode == 0, out.stderr[-3000:]
    return [ln for ln in out.stdout.splitlines() if ln.strip()]


def test_reference_arm_line():
    lines = run_bench(["--impl", "reference", "--config", "C1", "--steps", "2", "--warmup", "1"])
    assert len(lines) == 1
    d = json.loads(lines[0])
    assert d["impl"] == "reference" and d["unit"] == "events/s" and d["higher_is_better"] is True
    assert d["value"] > 0 and d["steps"] == 2 and d["warmup"] == 1
    cb = d["cpu_baseline"]
    assert cb["kind"] == "oracle" and cb["cores"] >= 1 and cb["value"] == d["value"] and cb["sample"]
    assert d["e2e"] == {"value": d["value"], "unit": "events/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}
    assert d["config"]["workload"].startswith("C1")
    assert d["config"]["workload"] == repo_arm_workload("C1")  # the same workload string as the repo arm
    assert d["config"]["sample_events_per_step"] > 0


def repo_arm_workload(name):
    import importlib.util
    import lmgen
    spec = importlib.util.spec_from_file_location("bench_mod", BENCH)
    m = importlib.util.module_from_spec(spec)
    spec.loader.exec_module(m)
    return m.workload(lmgen.CONFIGS[name])


def test_reference_arm_other_ranks_are_silent():
    lines = run_bench(["--impl", "reference", "--config", "C1", "--steps", "1", "--warmup", "1"],
                      env={"RANK": "1", "WORLD_SIZE": "2", "LOCAL_RANK": "1"})
    assert lines == []


@pytest.mark.gpu
def test_cuda_arm_line():
    torch = pytest.importorskip("torch")
    if not torch.cuda.is_available():
        pytest.skip("needs a GPU")
    lines = run_bench(["--config", "C1", "--steps", "4", "--warmup", "3", "--cpu-sample", "2000"])
    d = json.loads(lines[-1])
    for k in ("metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better", "scaling",
              "vs_baseline", "dtype", "data", "config", "roofline", "cpu_baseline", "e2e", "gpu_launches", "clocks"):
        assert k in d, k
    assert d["n_gpus"] == 1 and d["steps"] == 4 and d["warmup"] == 3 and d["value"] > 0
    r = d["roofline"]
    for k in ("bound", "achieved", "peak", "unit", "frac", "traffic"):
        assert k in r, k
    assert r["achieved"] > 0 and r["peak"] > 0 and abs(r["frac"] - r["achieved"] / r["peak"]) < 1e-9
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["cores"] >= 1
    e = d["e2e"]
    assert e["value"] > 0 and e["h2d_bytes_per_step"] > 0 and e["d2h_bytes_per_step"] > 0
    # one f -> brick conversion per reconstruct call, then (projection, update) per subset
    assert d["gpu_launches"] >= 2 * d["steps"]
    assert "sm_mhz" in d["clocks"] and "reasons" in d["clocks"]
    assert d["config"]["workload"] == repo_arm_workload("C1")
    rs = d["roofline_step"]
    assert rs["t_roof_ms"] > 0 and abs(rs["frac"] - rs["t_roof_ms"] / rs["t_meas_ms"]) < 1e-9
    assert rs["terms_ms"]["combine_t_ar_roof"] == 0.0  # one GPU: no combine
    m = d["p8_share_model"]
    assert m["P"] == 8 and m["fused"]["step_ms"] > m["project_share_ms"]
