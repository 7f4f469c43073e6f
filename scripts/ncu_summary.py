"""Summarise an ncu --csv launch list (gpu__time_duration.sum): per-kernel count, total, mean, share."""
import collections
import csv
import sys


def main(path):
    hdr = None
    tot = collections.defaultdict(float)
    cnt = collections.Counter()
    for r in csv.reader(open(path)):
        if "Kernel Name" in r:
            hdr = r
            continue
        if not hdr or len(r) != len(hdr):
            continue
        d = dict(zip(hdr, r))
        if d.get("Metric Name") != "gpu__time_duration.sum":
            continue
        nm = d["Kernel Name"].split("(")[0].split("<")[0]
        v = float(d["Metric Value"].replace(",", ""))
        scale = {"nsecond": 1e-3, "ns": 1e-3, "usecond": 1.0, "us": 1.0, "msecond": 1e3, "ms": 1e3}
        v *= scale.get(d["Metric Unit"], 1e-3)
        tot[nm] += v
        cnt[nm] += 1
    total = sum(tot.values())
    for k, v in sorted(tot.items(), key=lambda x: -x[1]):
        print(f"{k:40s} {cnt[k]:5d} {v:12.1f} us {v / cnt[k]:10.2f} us/launch {100 * v / total:5.1f}%")
    print(f"total {total:.1f} us")


if __name__ == "__main__":
    main(sys.argv[1])
