"""Per-launch table from an `ncu --metrics ... --csv` log (one row per launch)."""
import collections
import csv
import sys


def table(path, first=None, count=None):
    lines = [l for l in open(path) if l.startswith('"')]
    rows = list(csv.DictReader(lines))
    by = collections.OrderedDict()
    for r in rows:
        by.setdefault((r["ID"], r["Kernel Name"].split("(")[0]), {})[r["Metric Name"]] = r["Metric Value"]
    items = list(by.items())
    if first is not None:
        items = items[first:first + (count or len(items))]
    tot = 0.0
    for (_, name), m in items:
        t = float(m["gpu__time_duration.sum"]) / 1e3
        tot += t
        extra = " ".join(f"{k.split('__')[1][:18]}={m[k]}" for k in m if k != "gpu__time_duration.sum")
        print(f"{name:28s} {t:9.1f} us  {extra}")
    print(f"total {tot:.1f} us over {len(items)} launches")


if __name__ == "__main__":
    table(sys.argv[1], *(int(a) for a in sys.argv[2:]))
