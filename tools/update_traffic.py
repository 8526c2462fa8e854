#!/usr/bin/env python
"""Writes profiles/r01_traffic.json (read by bench.py) from one ncu --set full capture of
the C2 projection: DRAM bytes and L2 sectors (gathers, REDs) per launch.
Usage: update_traffic.py REPORT.ncu-rep SUMMARY_NAME"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def main(rep, summary):
    raw = list(csv.reader(io.StringIO(subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"],
                                                     capture_output=True, text=True).stdout)))
    names, units, row = raw[0], raw[1], raw[2]
    val = dict(zip(names, row))
    unit = dict(zip(names, units))

    def num(k):
        v = float(val[k].replace(",", ""))
        return v * {"Gbyte": 1e9, "Mbyte": 1e6, "Kbyte": 1e3, "byte": 1.0}.get(unit[k], 1.0)

    out = {"C2": {
        "kernel": "k_project<0>",
        "dram_bytes_read_per_launch": int(num("dram__bytes_read.sum")),
        "dram_bytes_write_per_launch": int(num("dram__bytes_write.sum")),
        "note": "one ncu --set full capture (-s 3 -c 1) of python bench.py --steps 3 --warmup 3 --no-cpu-baseline "
                "--no-e2e; L2 flushed before the step, so this is the cold refill of the brick images (2 x 27 MB) plus "
                "the 24 MB event stream; l2 sectors = lts__t_sectors_srcunit_tex_op_read/red.sum",
        "source": f"profiles/{summary}",
        "l2_sectors_read_per_launch": int(num("lts__t_sectors_srcunit_tex_op_read.sum")),
        "l2_sectors_red_per_launch": int(num("lts__t_sectors_srcunit_tex_op_red.sum")),
    }}
    with open(os.path.join(ROOT, "profiles", "r01_traffic.json"), "w") as fh:
        json.dump(out, fh, indent=1)
    print(json.dumps(out, indent=1))


if __name__ == "__main__":
    main(sys.argv[1], sys.argv[2])
