#!/usr/bin/env python
"""Writes one config's entry of profiles/r02_traffic.json (read by bench.py) from an ncu
--set full capture of that config's projection: DRAM bytes and L2 sectors (gathers, REDs)
per launch of the fused kernel, or summed over the launches of one subset step (the C4
z-slab form: 3 pass-A + 3 pass-B launches).
The listed z-slab form (C4: 3 pass-A + fine-window + 3 pass-B launches over k_zclass's lists)
is marked form = "listed".
Usage: update_traffic.py REPORT.ncu-rep SUMMARY_NAME [CONFIG] [LAUNCHES_PER_STEP] [FORM]"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
PATH = os.environ.get("LMOSEM_TRAFFIC_JSON") or os.path.join(ROOT, "profiles", "r02_traffic.json")


def main(rep, summary, config="C2", per_step=1, form=None):
    raw = list(csv.reader(io.StringIO(subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"],
                                                     capture_output=True, text=True).stdout)))
    names, units, rows = raw[0], raw[1], raw[2:]
    rows = rows[:per_step]
    assert len(rows) == per_step, f"{len(rows)} launches in the report, need {per_step}"

    def num(row, k):
        val = dict(zip(names, row))
        unit = dict(zip(names, units))
        v = float(val[k].replace(",", ""))
        return v * {"Gbyte": 1e9, "Mbyte": 1e6, "Kbyte": 1e3, "byte": 1.0}.get(unit[k], 1.0)

    def tot(k):
        return int(sum(num(r, k) for r in rows))

    kernels = sorted({dict(zip(names, r)).get("Kernel Name", "?").split("(")[0] for r in rows})
    entry = {
        "kernel": ", ".join(kernels),
        "form": form,
        "launches_per_step": per_step,
        "dram_bytes_read_per_launch": tot("dram__bytes_read.sum"),
        "dram_bytes_write_per_launch": tot("dram__bytes_write.sum"),
        "note": f"ncu --set full capture of python bench.py --config {config} (--steps 3 --warmup 3 "
                "--no-cpu-baseline --no-e2e); per launch = summed over the launches of one subset step; ncu flushes "
                "L2 before each launch, so DRAM bytes are the cold refill of the images plus the event stream; l2 "
                "sectors = lts__t_sectors_srcunit_tex_op_read/red.sum",
        "source": f"profiles/{summary}",
        "l2_sectors_read_per_launch": tot("lts__t_sectors_srcunit_tex_op_read.sum"),
        "l2_sectors_red_per_launch": tot("lts__t_sectors_srcunit_tex_op_red.sum"),
        "l2_requests_read_per_launch": tot("lts__t_requests_srcunit_tex_op_read.sum"),
        "l2_requests_red_per_launch": tot("lts__t_requests_srcunit_tex_op_red.sum"),
        "req_cycles_active_pct": round(sum(num(r, "l1tex__m_l1tex2xbar_req_cycles_active.avg.pct_of_peak_sustained_elapsed")
                                           for r in rows) / len(rows), 2),
    }
    try:
        with open(PATH) as fh:
            out = json.load(fh)
    except (OSError, ValueError):
        out = {}
    out[config] = entry
    with open(PATH, "w") as fh:
        json.dump(out, fh, indent=1)
    print(json.dumps({config: entry}, indent=1))


if __name__ == "__main__":
    main(sys.argv[1], sys.argv[2], *(sys.argv[3:4]), *(int(x) for x in sys.argv[4:5]), *(sys.argv[5:6]))
