"""Average duration per kernel of an `ncu --metrics gpu__time_duration.sum --csv` launch list."""
import csv
import sys

for f in sys.argv[1:]:
    hdr, tot = None, {}
    for r in csv.reader(open(f)):
        if r and r[0] == "ID":
            hdr = r
            continue
        if hdr and len(r) == len(hdr):
            d = dict(zip(hdr, r))
            tot.setdefault(d["Kernel Name"].split("(")[0][:60], []).append(float(d["Metric Value"].replace(",", "")))
    print(f)
    for k, v in tot.items():
        print(f"  {k:60s} n={len(v):3d} avg={sum(v) / len(v) / 1e3:9.1f} us")
