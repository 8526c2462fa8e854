#!/usr/bin/env python
"""Summarise an ncu report: the 'details' page (section / metric / value) per kernel,
plus a few raw counters. Usage: ncu_summary.py REPORT.ncu-rep [raw-metric-regex ...]"""
import csv
import io
import re
import subprocess
import sys

RAW = [r"dram__bytes_(read|write)\.sum$", r"lts__t_sectors_op_(red|atom|read|write)\.sum$",
       r"lts__t_sectors\.sum$", r"lts__t_requests_op_red\.sum$", r"sm__inst_issued\.avg\.pct_of_peak_sustained_active$",
       r"sm__warps_active\.avg\.pct_of_peak_sustained_active$", r"launch__registers_per_thread$",
       r"gpu__time_duration\.sum$", r"l1tex__t_sectors_pipe_lsu_mem_global_op_ld\.sum$",
       r"l1tex__t_requests_pipe_lsu_mem_global_op_ld\.sum$", r"l1tex__t_sectors_pipe_lsu_mem_global_op_red\.sum$",
       r"l1tex__t_requests_pipe_lsu_mem_global_op_red\.sum$", r"lts__t_sector_hit_rate\.pct$",
       r"sm__pipe_fp64_cycles_active\.avg\.pct_of_peak_sustained_active$", r"smsp__inst_executed\.sum$",
       r"lts__throughput\.avg\.pct_of_peak_sustained_elapsed$", r"l1tex__t_sector_hit_rate\.pct$",
       r"lts__t_sectors_srcunit_tex_op_read\.sum$", r"lts__t_sectors_srcunit_tex_op_red\.sum$"]


def run(args):
    return subprocess.run(["ncu", "-i"] + args, capture_output=True, text=True).stdout


def main():
    rep = sys.argv[1]
    extra = sys.argv[2:]
    det = list(csv.reader(io.StringIO(run([rep, "--page", "details", "--csv"]))))
    h = det[0]
    ix = {k: h.index(k) for k in ("Kernel Name", "Section Name", "Metric Name", "Metric Unit", "Metric Value")}
    cur = None
    for r in det[1:]:
        if len(r) <= ix["Metric Value"] or not r[ix["Metric Name"]]:
            continue
        k = r[ix["Kernel Name"]][:80]
        if k != cur:
            print(f"\n## {k}")
            cur = k
        print(f"  {r[ix['Section Name']][:28]:28s} | {r[ix['Metric Name']][:44]:44s} | {r[ix['Metric Value']]:>14s} {r[ix['Metric Unit']]}")
    raw = list(csv.reader(io.StringIO(run([rep, "--page", "raw", "--csv"]))))
    if raw:
        names, units = raw[0], raw[1]
        pats = [re.compile(p) for p in RAW + extra]
        print("\n## raw counters")
        for row in raw[2:]:
            for n, u, v in zip(names, units, row):
                if any(p.search(n) for p in pats):
                    print(f"  {n:70s} {v:>18s} {u}")


if __name__ == "__main__":
    main()
