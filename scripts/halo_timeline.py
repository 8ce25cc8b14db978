"""Halo-overlap timeline on the NCCL path in loopback (N = 1, faces through NCCL to
self): CUDA events on both streams around the pack, the exchange and the interior / boundary
kernels of the Dslash (qudax_halo_timeline).  Prints one JSON line per precision: the median over
the recorded Mhat applications of each mark (µs from the start of the second Dslash of Mhat) and
the overlap = the part of the comm-stream work (pack + exchange) that ran while the interior
kernel ran.

    python scripts/halo_timeline.py [--dims 32,32,32,64]
"""
import argparse
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import qgen  # noqa: E402
from paper_1011_0024_b200 import qudax  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--dims", default="32,32,32,64")
    ap.add_argument("--reps", type=int, default=20)
    args = ap.parse_args()
    dims = tuple(int(v) for v in args.dims.split(","))
    U = qgen.gauge(dims, 1005, eps=0.1)
    psi = qgen.spinor(dims, 2005)
    for prec, recon in ((4, 12), (2, 12), (8, 18)):
        ctx = qudax.Context(dims, comm=qudax.COMM_NCCL, nccl_id=qudax.nccl_unique_id(), overlap=True)
        ctx.gauge_load(U, 0.124, 1.0, prec=prec, recon=recon)
        fi, fo = ctx.new_field(prec), ctx.new_field(prec)
        ctx.spinor_load(fi, prec, 0, psi)
        for _ in range(3):
            ctx.matpc(fo, fi, prec)
        ctx.halo_timeline(True)
        marks = []
        for _ in range(args.reps):
            ctx.matpc(fo, fi, prec)
            marks.append(ctx.halo_timeline(True, read=True))
        ctx.halo_timeline(False)
        med = {k: statistics.median(m[k] for m in marks) for k in marks[0]}
        comm0, comm1 = med["pack_start"], med["exchange_end"]
        int0, int1 = med["interior_start"], med["interior_end"]
        overlap = max(0.0, min(comm1, int1) - max(comm0, int0))
        print(json.dumps({"prec": prec, "recon": recon, "dims": dims, "median_marks_us": med,
                          "comm_stream_us": comm1 - comm0, "interior_us": int1 - int0,
                          "overlap_us": overlap, "exchange_hidden": comm1 <= int1}), flush=True)
        ctx.close()


if __name__ == "__main__":
    main()
