"""Summarise an ncu --csv metrics log: one line per launch (time, DRAM bytes, GB/s)."""
import collections
import csv
import io
import sys


def load(path):
    txt = open(path).read().splitlines()
    start = next(i for i, l in enumerate(txt) if l.startswith('"ID"'))
    rows = list(csv.DictReader(io.StringIO("\n".join(txt[start:]))))
    k = collections.OrderedDict()
    for r in rows:
        d = k.setdefault(r["ID"], {"name": r["Kernel Name"], "grid": r["Grid Size"], "block": r["Block Size"]})
        try:
            d[r["Metric Name"]] = float(r["Metric Value"].replace(",", ""))
        except ValueError:
            d[r["Metric Name"]] = r["Metric Value"]
    return k


def main(path):
    for i, d in load(path).items():
        t = d.get("gpu__time_duration.sum", 0.0)
        rd = d.get("dram__bytes_read.sum", 0.0)
        wr = d.get("dram__bytes_write.sum", 0.0)
        name = d["name"].split("(")[0][:48]
        print(f"{i:>4} {name:48s} grid {d['grid']:>14} blk {d['block']:>12} {t / 1e3:10.2f} us  rd {rd / 1e6:10.2f} MB"
              f"  wr {wr / 1e6:8.2f} MB  {(rd + wr) / t if t else 0:8.1f} GB/s")


if __name__ == "__main__":
    main(sys.argv[1])
