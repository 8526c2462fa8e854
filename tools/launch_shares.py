#!/usr/bin/env python
"""Per-kernel totals and shares of an ncu launch list (--metrics gpu__time_duration.sum --csv)."""
import csv
import sys
from collections import defaultdict


def main(path):
    h, t, n = None, defaultdict(float), defaultdict(int)
    for r in csv.reader(open(path)):
        if "Kernel Name" in r:
            h = r
            continue
        if h and len(r) == len(h):
            d = dict(zip(h, r))
            if d.get("Metric Name") == "gpu__time_duration.sum":
                k = d["Kernel Name"].split("(")[0]
                t[k] += float(d["Metric Value"])
                n[k] += 1
    tot = sum(t.values())
    ours = sum(v for k, v in t.items() if "lmk::" in k)
    print(f"{'kernel':60s} {'launches':>8s} {'total ms':>9s} {'share':>6s} {'of lmk::':>8s}")
    for k in sorted(t, key=lambda k: -t[k]):
        own = f"{100 * t[k] / ours:7.1f}%" if "lmk::" in k else ""
        print(f"{k:60s} {n[k]:8d} {t[k] / 1e6:9.3f} {100 * t[k] / tot:5.1f}% {own:>8s}")


if __name__ == "__main__":
    main(sys.argv[1])
