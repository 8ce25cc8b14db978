"""Opcode mix of an ncu --page source --csv (SASS) dump: warp-level instructions executed and
stall samples per opcode.   python scripts/sass_mix.py <source.csv> [top]"""
import collections
import csv
import sys

rows = list(csv.reader(open(sys.argv[1])))
hdr = rows[1]
si, ie, ss = hdr.index("Source"), hdr.index("Instructions Executed"), hdr.index("Warp Stall Sampling (All Samples)")
inst, samp = collections.Counter(), collections.Counter()
for r in rows[2:]:
    if len(r) <= ie:
        continue
    op = r[si].split()
    if not op:
        continue
    o = op[0]
    if o.startswith("@"):
        o = op[1]
    o = o.split(".")[0]
    inst[o] += float(r[ie] or 0)
    samp[o] += float(r[ss] or 0)
ti, ts = sum(inst.values()), sum(samp.values())
print(f"total warp instructions {ti:.0f}, stall samples {ts:.0f}")
for o, v in inst.most_common(int(sys.argv[2]) if len(sys.argv) > 2 else 30):
    print(f"{o:10s} {v:12.0f} {100 * v / ti:6.2f}%  samples {100 * samp[o] / ts:6.2f}%")
