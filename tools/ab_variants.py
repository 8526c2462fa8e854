#!/usr/bin/env python
"""A/B kernel variants: `build` compiles each variant (here, CPU) into variants/;
`run` benchmarks each on the GPU (LMOSEM_LIB=<variant> python bench.py ...)."""
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
VARIANTS = {
    # compile-time switches left in the kernel: LMK_CTA_THREADS, LMK_MIN_BLOCKS
    # (rejected variants are listed with their numbers in DESIGN.md §7)
    "default": [],
    "setup_only": ["LMK_SETUP_ONLY=1"],
    "append2": ["LMK_APPEND2=1"],  # two-ballot path-buffer prefix
    "unroll1": ["LMK_GEOM_UNROLL=1"],
    "unroll3": ["LMK_GEOM_UNROLL=3"],
    "unroll4": ["LMK_GEOM_UNROLL=4"],  # diagnostic: claims + tiles + float64 setup, no traversal
    "c256x2": ["LMK_MIN_BLOCKS=2"],
    "slab4": ["LMK_SLAB_MIN_BLOCKS=4"],
    "guided1": ["LMOSEM_GUIDED_LARGE=1", "LMOSEM_GUIDED_SMALL=1"],
    "guided2": ["LMOSEM_GUIDED_LARGE=2", "LMOSEM_GUIDED_SMALL=2"],
    "guided3": ["LMOSEM_GUIDED_LARGE=3", "LMOSEM_GUIDED_SMALL=3"],
    "guided4": ["LMOSEM_GUIDED_LARGE=4", "LMOSEM_GUIDED_SMALL=4"],
    "fixed": ["LMOSEM_GUIDED_LARGE=0", "LMOSEM_GUIDED_SMALL=0"],
    "nostatic": ["LMOSEM_STATIC_BATCH=0"],
    "min2": ["LMOSEM_MIN_BATCH=2"],
    "claims8": ["LMOSEM_CLAIMS=8", "LMOSEM_MIN_BATCH=2"],
    "claims2": ["LMOSEM_CLAIMS=2"],
    "read1": ["LMOSEM_READ_THREADS=1"],
    "read2": ["LMOSEM_READ_THREADS=2"],
    "read3": ["LMOSEM_READ_THREADS=3"],
    "read4": ["LMOSEM_READ_THREADS=4"],
    "read6": ["LMOSEM_READ_THREADS=6"],
    "read16": ["LMOSEM_READ_THREADS=16"],
}


def build(names):
    from paper_conf_ipps_steuwerkg12_b200 import build as b
    for n in names:
        out = os.path.join(ROOT, "variants", f"liblmosem_{n}.so")
        b.build(defines=VARIANTS[n], out=out)
        print("built", out)


def run(names, extra):
    res = {}
    for n in names:
        env = dict(os.environ, LMOSEM_LIB=os.path.join(ROOT, "variants", f"liblmosem_{n}.so"))
        out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--no-cpu-baseline", "--no-e2e",
                              "--steps", "40", "--warmup", "5", *extra], env=env, capture_output=True, text=True)
        try:
            d = json.loads(out.stdout.strip().splitlines()[-1])
            res[n] = {"events_per_s": d["value"], "project_ms": d["phase_ms_per_step"]["project"]}
        except Exception as e:  # noqa: BLE001
            res[n] = {"error": str(e), "stderr": out.stderr[-500:]}
        print(n, res[n], flush=True)
    return res


if __name__ == "__main__":
    names = [a for a in sys.argv[2:] if not a.startswith("--")] or list(VARIANTS)
    extra = [a for a in sys.argv[2:] if a.startswith("--")]
    if sys.argv[1] == "build":
        build(names)
    else:
        r = run(names, [x for e in extra for x in e.split("=", 1)])
        os.makedirs(os.path.join(ROOT, "gpurun_out"), exist_ok=True)
        with open(os.path.join(ROOT, "gpurun_out", "ab.json"), "w") as fh:
            json.dump(r, fh, indent=1)
