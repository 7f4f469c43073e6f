"""ncu launch list (gpu__time_duration.sum, --csv) -> per-kernel table for profiles/ (our kernels only)."""
import collections
import csv
import sys


def main(path, steps, header):
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
        nm = d["Kernel Name"].split("(")[0]
        if "rs::" not in nm and "kernel" not in nm:
            continue
        v = float(d["Metric Value"].replace(",", ""))
        v *= {"nsecond": 1e-6, "ns": 1e-6, "usecond": 1e-3, "us": 1e-3, "msecond": 1.0, "ms": 1.0}.get(d["Metric Unit"], 1e-6)
        tot[nm] += v
        cnt[nm] += 1
    total = sum(tot.values())
    print(header)
    print(f"# our kernels: {sum(cnt.values())} launches over {steps} approximations, {total:.2f} ms total device time")
    print("kernel,launches,total_ms,ms_per_approx,share_of_our_time")
    for k, v in sorted(tot.items(), key=lambda x: -x[1]):
        print(f"{k},{cnt[k]},{v:.4f},{v / steps:.4f},{v / total:.4f}")


if __name__ == "__main__":
    main(sys.argv[1], int(sys.argv[2]), sys.argv[3] if len(sys.argv) > 3 else "")
