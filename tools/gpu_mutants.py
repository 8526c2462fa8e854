#!/usr/bin/env python
"""Mutation check of the GPU parity tests: copies of the CUDA sources, each with one
plausible kernel bug, are built here (`build`, nvcc cross-compiles) and run on the B200
(`run`) against a fast subset of tests/test_parity_gpu.py with LMOSEM_LIB pointing at the
mutant. A mutant the parity tests do not catch is reported as SURVIVED (diagnostic; the
results are in profiles/r01_gpu_mutants.txt).
Usage: python tools/gpu_mutants.py build|run [name-substring]"""
import json
import os
import shutil
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
CSRC = os.path.join(ROOT, "paper_conf_ipps_steuwerkg12_b200", "csrc")
OUT = os.path.join(ROOT, "variants", "mutants")
K = "lmosem_kernels.cuh"
H = "lmosem.cu"
# (name, file, original, mutated, replace_all)
MUTANTS = [
    ("piece 1 from the later crossing", K, "P.j1 = Ja + ((db <= dc) ? (Jb1 + Jc0) : (Jb0 + Jc1));",
     "P.j1 = Ja + ((db <= dc) ? (Jb0 + Jc1) : (Jb1 + Jc0));", False),
    ("first-slab float64 clip lengths not used", K, "if (decltype(first)::value && k == 0) {",
     "if (false && k == 0) {", False),
    ("last-slab float64 clip lengths not used", K, "if (decltype(last)::value && k == L.ns - 1) {",
     "if (false && k == L.ns - 1) {", False),
    ("last slab takes the first slab's clip lengths", K, "P.l0 = lds1(clip_l + 12u);", "P.l0 = lds1(clip_l);", False),
    ("z-slab LOR record: slopes b and c swapped on load", K,
     '"=l"(L.sb), "=l"(L.sc) : "r"(a + 16u)', '"=l"(L.sc), "=l"(L.sb) : "r"(a + 16u)', False),
    ("z-slab LOR record: clip lengths read 4 bytes off", K, "constexpr unsigned kClipOff = kLorSmem ? 56u : 0u;",
     "constexpr unsigned kClipOff = kLorSmem ? 52u : 0u;", False),
    ("fp without mm per slab unit", K, "fpv = warp_sum(acc) * L.lunit;",
     "fpv = warp_sum(acc);", False),
    ("back-projected weight without mm per slab unit", K,
     "const float inv = L.lunit / fpv;", "const float inv = 1.0f / fpv;", False),
    ("texture gather of piece 0 reads piece 1's voxel", K,
     "acc = fmaf(v0 ? tex1Dfetch<float>(g.tex_fb, P.j0) : 0.f, P.l0, acc);",
     "acc = fmaf(v0 ? tex1Dfetch<float>(g.tex_fb, P.j1) : 0.f, P.l0, acc);", False),
    ("LSU gather of piece 2 dropped (MODE 0 / z-slab pass A)", K,
     "acc = fmaf(v2 ? __ldg(fb + P.j2) : 0.f, P.l2, acc);", "acc = acc;", False),
    ("RED without 1/fp", K, "atomicAdd(cb + q.x, __int_as_float(q.y) * inv);", "atomicAdd(cb + q.x, __int_as_float(q.y));",
     False),
    ("fp <= 0 events not skipped", K, "if (kScatter && fpv > 0.0f) {", "if (kScatter) {", False),
    ("fraction converted from its high bits only", K,
     "return __ull2float_rn(((unsigned long long)(hi & ((1u << (FIX_BITS - 32)) - 1u)) << 32) | lo);",
     "return __ull2float_rn(((unsigned long long)(hi & ((1u << (FIX_BITS - 32)) - 1u)) << 32) | (lo & 0xff000000u));",
     False),
    ("halo of one minor axis missing", K, "+ HALO_LO * (W.Ab + W.Ac);", "+ HALO_LO * W.Ab;", False),
    ("update without the norm", K, "return (c > 0.0f && s > 0.0f) ? f * __fdiv_rn(c, s) : f;",
     "return (c > 0.0f && s > 0.0f) ? f * c : f;", False),
    ("update without the c > 0 guard", K, "return (c > 0.0f && s > 0.0f) ? f * __fdiv_rn(c, s) : f;",
     "return (s > 0.0f) ? f * __fdiv_rn(c, s) : f;", False),
    ("c not re-zeroed by the update", K, "        F[1] = f1;\n        C[0] = make_float4(0.f, 0.f, 0.f, 0.f);\n"
     "        C[1] = make_float4(0.f, 0.f, 0.f, 0.f);", "        F[1] = f1;", False),
    ("events shifted by one", K, "const int64_t idx = base + lane;", "const int64_t idx = base + lane + 1;", False),
    ("last 16 bytes of an event tile not staged", K, "for (int q = lane; q < (3 * m) / 2; q += 32)",
     "for (int q = lane; q < (3 * m) / 2 - 1; q += 32)", False),
    ("dominant axis not the largest", K, "const int a = (ax >= ay && ax >= az) ? 0 : ((ay >= az) ? 1 : 2);",
     "const int a = (ax >= ay) ? 0 : ((ay >= az) ? 1 : 2);", False),
    ("stationary-axis voxel row by multiplication with 1/v", K,
     "        if (d[k] == 0.0) u1[k] = (p1[k] - g.lo[k]) / g.v[k];\n", "", False),
    ("brick voxel order x/y swapped", K, "2 * bx + (q & 1), 2 * by + ((q >> 1) & 1)",
     "2 * bx + ((q >> 1) & 1), 2 * by + (q & 1)", True),
    ("PDL: no wait before the first image access", K, "            pdl_wait();\n            dep_ready = true;",
     "            dep_ready = true;", False),
    ("z-slab boundaries off by one brick", H, "g.clo[a] = 2 * (int)((int64_t)half * k / K);",
     "g.clo[a] = 2 * (int)((int64_t)half * k / K) + (k > 0 ? 2 : 0);", False),
    # the multi-rank combine (round 2: caught by tests/test_loopback_gpu.py, P ranks on one GPU)
    ("combine: events not block-split (every rank projects the whole subset)", H,
     "if (whole_subset) block_range(n, ctx->rank, ctx->world, &b, &e);", "if (false) block_range(n, ctx->rank, ctx->world, &b, &e);", False),
    ("combine: ISD block offset ignores the rank", H, "b0 = chunk * ctx->rank;", "b0 = 0;", True),
    ("combine: reduce-scatter count in bricks, not floats", H, "coll_reduce_scatter(ctx, ctx->c, my_c, (size_t)(8 * chunk))",
     "coll_reduce_scatter(ctx, ctx->c, my_c, (size_t)(chunk))", False),
    ("combine: ISD update leaves the other ranks' partial c (no zero_to)", H,
     "launch_update(ctx, nullptr, blk_b, blk_e, alloc)", "launch_update(ctx, nullptr, blk_b, blk_e)", True),
    ("combine: ISD all-gather of f dropped", H,
     "        if ((s = coll_all_gather(ctx, ctx->fb + 8 * b0, ctx->fb, (size_t)(8 * chunk)))) return s;\n", "", False),
    ("combine: all-reduce over a brick count", H, "coll_all_reduce(ctx, ctx->c, (size_t)ctx->nbf)",
     "coll_all_reduce(ctx, ctx->c, (size_t)ctx->bricks.nb)", True),
    ("fused combine: every rank takes rank 0's block", K, "const int64_t b0 = chunk * team.rank(), b1",
     "const int64_t b0 = chunk * 0, b1", False),
    ("fused combine: the last real brick column treated as halo", K, "bx < (unsigned)it.rhi[0]",
     "bx + 1 < (unsigned)it.rhi[0]", False),
    ("fused combine: local c not re-zeroed", K, "            C[2 * b] = z;\n            C[2 * b + 1] = z;\n", "", False),
    ("fused combine: second brick of a pair not stored", K, "            team.store_f(ob, nb0, nb1);\n", "", False),
    # the listed z-slab form (round 2: caught by tests/test_zlist_gpu.py and the loopback test)
    ("listed: window membership without its margin", K, "if (zl >= lo + m && zh <= lo + w - m) return j;",
     "if (zl >= lo - m && zh <= lo + w + m) return j;", False),
    ("listed: coarse membership shrunk by the margin", K,
     "if (zh + m > (float)zc.cb[k] && zl - m < (float)zc.cb[k + 1]) {",
     "if (zh > (float)zc.cb[k] + m && zl < (float)zc.cb[k + 1] - m) {", False),
    ("listed: window LORs also in the coarse lists", K, "if (jf >= 0) return zlist_code(zc.K + jf, 1);",
     "if (jf >= 0) return zlist_code(0, zc.K + jf + 1);", False),
    ("listed: medium-window LORs in no list", K, "if (jm >= 0) return zlist_code(zc.K + zc.Kf + jm, 1);",
     "if (jm >= 0) return 0u;", False),
    ("listed: medium window of the next family index", K, "if (jm >= 0) return zlist_code(zc.K + zc.Kf + jm, 1);",
     "if (jm >= 0) return zlist_code(zc.K + zc.Kf + min(jm + 1, zc.Km - 1), 1);", False),
    ("listed: list slots without the per-event offset", K,
     "if (q < cnt) lists[(int64_t)(l0 + q) * cap + s_base[l0 + q] + off[p][q]] = e;",
     "if (q < cnt) lists[(int64_t)(l0 + q) * cap + s_base[l0 + q]] = e;", False),
    ("listed: segment lookup off by one", K, "while (sg < la.nseg - 1 && idx >= s_segend[sg])",
     "while (sg < la.nseg - 1 && idx > s_segend[sg])", False),
    ("listed: window box not applied per event", K, "const bool w = LIST && la.box && k == la.axis;",
     "const bool w = false;", False),
]
# Not listed: equivalent mutants. A medium-window LOR also put in every coarse list is
# projected twice in pass A (its whole path in the window, its pieces per slab: fp doubles) and
# back-projected twice with that fp, so c is unchanged (measured: it survives, as expected). Dropping the 2^-40 offset of the mirrored frame changes
# only exactly integral up-moving positions, where "voxel m - 1 with a crossing at d = 0"
# yields the same pieces as "voxel m, no crossing" (the zero-length piece is dropped); and
# any change to the ISD rank block (b0 = chunk * rank) is invisible at world size 1, the only
# one a single GPU can run (NCCL refuses two ranks on one GPU; the block split itself is
# covered by the gloo tests and the emulated-rank combine test). The z-slab pass B setup
# test `ok && fp_known > 0` only saves work: the back-projection's own fp > 0 guard skips
# the same events (measured: the mutant passes every parity test, as expected).
TESTS = ("listed or loopback_c1 or loopback_c2 or loopback_ragged or golden or degenerate or axis_parallel or c1_ or zslab_passes_match_oracle_c1 or odd_extents or "
         "lors_in_voxel_faces or one_subset_paper_shaped or programmatic or nccl_combine_single_rank or "
         "combine_modes_single_rank or zero_forward_projection or lsu_and_texture")


def _selected(name, only):
    return only is None or name == "control" or only in name


def build(only=None):
    from paper_conf_ipps_steuwerkg12_b200 import build as b
    os.makedirs(OUT, exist_ok=True)
    names = [("control", None, None, None, False)] + MUTANTS
    for i, (name, fn, old, new, every) in enumerate(names):
        if not _selected(name, only):
            continue
        if os.environ.get("MUTANTS_KEEP") and os.path.exists(os.path.join(OUT, f"liblmosem_m{i}.so")):
            continue  # resume a partial build
        d = os.path.join(OUT, f"src{i}")
        shutil.rmtree(d, ignore_errors=True)
        shutil.copytree(CSRC, d)
        if fn:
            p = os.path.join(d, fn)
            s = open(p).read()
            n = s.count(old)
            assert n >= 1 and (every or n == 1), f"{name}: pattern occurs {n} times"
            open(p, "w").write(s.replace(old, new))
        b.build(out=os.path.join(OUT, f"liblmosem_m{i}.so"), csrc=d)
        print("built", i, name, flush=True)


def run(only=None):
    names = [("control", None, None, None, False)] + MUTANTS
    res = []
    for i, (name, *_rest) in enumerate(names):
        if not _selected(name, only):
            continue
        env = dict(os.environ, LMOSEM_LIB=os.path.join(OUT, f"liblmosem_m{i}.so"))
        out = subprocess.run([sys.executable, "-m", "pytest", os.path.join(ROOT, "tests", "test_parity_gpu.py"),
                              os.path.join(ROOT, "tests", "test_loopback_gpu.py"),
                              os.path.join(ROOT, "tests", "test_zlist_gpu.py"), "-x",
                              "-q", "-p", "no:cacheprovider", "-k", TESTS], capture_output=True, text=True, cwd=ROOT,
                             env=env, timeout=900)
        tail = [ln for ln in out.stdout.splitlines() if ln.startswith("FAILED") or " passed" in ln or " failed" in ln]
        ok = out.returncode == 0
        verdict = ("ok" if ok else "BROKEN") if i == 0 else ("SURVIVED" if ok else "killed")
        res.append({"mutant": name, "verdict": verdict, "evidence": tail[:2]})
        print(f"{verdict:9s} {name}: {tail[:1]}", flush=True)
    print(json.dumps(res, indent=1))


if __name__ == "__main__":
    {"build": build, "run": run}[sys.argv[1]](sys.argv[2] if len(sys.argv) > 2 else None)
