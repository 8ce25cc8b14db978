"""Mean per-kind timings of an ab_dslash.sh log: python scripts/ab_summary.py gpurun_out/TAG/ab.log"""
import collections
import json
import sys

rows = [json.loads(l) for l in open(sys.argv[1]) if l.startswith("{")]
acc = collections.defaultdict(list)
for r in rows:
    for k in ("hop", "clover_inv", "xpay", "inv_xpay"):
        acc[(r["case"], r["tag"], k)].append(r[k]["us"])
    for n in (4, 8):
        if f"matpc_x{n}" in r:
            acc[(r["case"], r["tag"], f"x{n}")].append(r[f"matpc_x{n}"]["us_per_rhs"])
print("case tag: hop / clover_inv / xpay / inv_xpay / Mhat-x8 per RHS (us)")
for c, t in sorted(set((a, b) for a, b, _ in acc)):
    print(c, t, " ".join("%.1f" % (sum(acc[(c, t, k)]) / len(acc[(c, t, k)])) for k in ("hop", "clover_inv", "xpay", "inv_xpay", "x8") if acc[(c, t, k)]))
