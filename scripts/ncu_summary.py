"""Summarise ncu output into profiles/ (run here, on the CPU box).

    python scripts/ncu_summary.py launches <launches.csv> <out.md>
    python scripts/ncu_summary.py full <prof.ncu-rep> <out.md> [--traffic-json profiles/dslash_traffic.json --lattice 32,32,32,64]
"""
import collections
import csv
import io
import json
import subprocess
import sys


def launches(path, out):
    rows = list(csv.reader(open(path)))
    h = next(i for i, r in enumerate(rows) if "Kernel Name" in r and "Metric Value" in r)
    hdr = rows[h]
    ki, vi, ui = hdr.index("Kernel Name"), hdr.index("Metric Value"), hdr.index("Metric Unit")
    tot, cnt = collections.defaultdict(float), collections.Counter()
    for r in rows[h + 1:]:
        if len(r) <= vi:
            continue
        v = float(r[vi].replace(",", ""))
        u = r[ui]
        v = v / 1000 if u in ("nsecond", "ns") else (v * 1000 if u in ("msecond", "ms") else v)
        name = r[ki].split("(")[0].replace("void ", "")
        tot[name] += v
        cnt[name] += 1
    T = sum(tot.values())
    lines = [f"# Launch list summary ({path})", "",
             "ncu `--metrics gpu__time_duration.sum --clock-control none` (cold-cache, serialised: compare shares).", "",
             f"Total {T:.1f} us over {sum(cnt.values())} launches.", "",
             "| share | total us | launches | avg us | kernel |", "|---:|---:|---:|---:|---|"]
    for k, v in sorted(tot.items(), key=lambda x: -x[1]):
        lines.append(f"| {v / T * 100:.2f}% | {v:.1f} | {cnt[k]} | {v / cnt[k]:.2f} | `{k}` |")
    open(out, "w").write("\n".join(lines) + "\n")
    print("\n".join(lines[:30]))


WANT = ["gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
        "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed", "dram__throughput.avg.pct_of_peak_sustained_elapsed",
        "launch__registers_per_thread", "launch__grid_size", "launch__block_size", "launch__occupancy_limit_registers",
        "sm__warps_active.avg.pct_of_peak_sustained_active", "lts__t_sector_hit_rate.pct", "l1tex__t_sector_hit_rate.pct",
        "sm__throughput.avg.pct_of_peak_sustained_elapsed", "smsp__inst_executed.sum", "lts__t_bytes.sum",
        "sm__inst_executed_pipe_lsu.avg.pct_of_peak_sustained_active",
        "smsp__average_warp_latency_issue_stalled_long_scoreboard.ratio",
        "smsp__warp_issue_stalled_long_scoreboard_per_warp_active.pct",
        "smsp__warp_issue_stalled_lg_throttle_per_warp_active.pct"]


def to_bytes(v, u):
    f = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "Tbyte": 1e12}
    return v * f.get(u, 1)


def full(path, out, traffic_json=None, lattice=None):
    raw = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(raw)))
    hdr, units = rows[0], rows[1]
    lines = [f"# ncu --set full summary ({path})", ""]
    per_kernel = collections.defaultdict(list)
    for r in rows[2:]:
        name = r[hdr.index("Kernel Name")]
        lines += [f"## `{name}`", "", "| metric | value | unit |", "|---|---:|---|"]
        for w in WANT:
            if w in hdr:
                i = hdr.index(w)
                lines.append(f"| {w} | {r[i]} | {units[i]} |")
        lines.append("")
        rd = to_bytes(float(r[hdr.index("dram__bytes_read.sum")]), units[hdr.index("dram__bytes_read.sum")])
        wr = to_bytes(float(r[hdr.index("dram__bytes_write.sum")]), units[hdr.index("dram__bytes_write.sum")])
        per_kernel[name].append(rd + wr)
    open(out, "w").write("\n".join(lines) + "\n")
    print("\n".join(lines))
    if traffic_json:
        d = {"source": path, "lattice": [int(x) for x in lattice.split(",")],
             "dram_bytes_per_launch_by_kernel": {k: sum(v) / len(v) for k, v in per_kernel.items()}}
        sel = [v for k, vs in per_kernel.items() if "<4, 12" in k for v in vs]
        d["dram_bytes_per_launch"] = sum(sel) / len(sel) if sel else None
        json.dump(d, open(traffic_json, "w"), indent=1)


if __name__ == "__main__":
    if sys.argv[1] == "launches":
        launches(sys.argv[2], sys.argv[3])
    else:
        tj = sys.argv[sys.argv.index("--traffic-json") + 1] if "--traffic-json" in sys.argv else None
        lat = sys.argv[sys.argv.index("--lattice") + 1] if "--lattice" in sys.argv else None
        full(sys.argv[2], sys.argv[3], tj, lat)
