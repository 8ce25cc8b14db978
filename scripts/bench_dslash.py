"""Dslash kernel micro-benchmark: per kind and precision, CUDA-event timed inside the library,
compulsory-byte GB/s against the measured HBM copy peak.  Used for kernel tuning experiments
(QUDAX_LIB selects a variant build).

    python scripts/bench_dslash.py [--dims 32,32,32,64] [--reps 50] [--cases f32-12,h-12,f64-18]
"""
import argparse
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np  # noqa: E402
import torch  # noqa: E402

import qgen  # noqa: E402
from paper_1011_0024_b200 import qudax  # noqa: E402

CASES = {"f64-18": (8, 18), "f64-12": (8, 12), "f32-18": (4, 18), "f32-12": (4, 12), "f32-8": (4, 8),
         "h-18": (2, 18), "h-12": (2, 12), "h-8": (2, 8)}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--dims", default="32,32,32,64")
    ap.add_argument("--reps", type=int, default=50)
    ap.add_argument("--cases", default="f32-12,h-12,f64-18")
    ap.add_argument("--tag", default=os.environ.get("QUDAX_LIB", "default"))
    ap.add_argument("--nrhs", default="", help="comma list: also time multi-RHS Mhat for these counts")
    ap.add_argument("--flags", type=int, default=0, help="qudax init flags (A/B of kernel variants)")
    args = ap.parse_args()
    dims = tuple(int(v) for v in args.dims.split(","))
    try:
        peak = json.load(open(os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                                           "MEASURED_PEAKS.json")))["hbm_gbs"]
    except OSError:  # driver-written per pod; else the profiling guide's fallback
        peak = 6650.0
    U = qgen.gauge(dims, 1005, eps=-1.0)
    psi = qgen.spinor(dims, 2005)
    ctx = qudax.Context(dims, flags=args.flags)
    for case in args.cases.split(","):
        prec, recon = CASES[case]
        ctx.gauge_load(U, 0.124, 1.0, prec=prec, recon=recon)
        fi, fo, fx = ctx.new_field(prec), ctx.new_field(prec), ctx.new_field(prec)
        ctx.spinor_load(fi, prec, 1, psi)
        ctx.spinor_load(fx, prec, 0, psi)
        res = {"case": case, "tag": args.tag, "dims": dims}
        for kind, name in ((0, "hop"), (1, "clover_inv"), (2, "xpay"), (3, "inv_xpay")):
            for _ in range(5):
                ctx.dslash(fo, fi, prec, 0, kind=kind, x=fx, a=-0.1)
            ctx.kernel_timing(True)
            for _ in range(args.reps):
                ctx.dslash(fo, fi, prec, 0, kind=kind, x=fx, a=-0.1)
            ks = ctx.kernel_stats()
            ctx.kernel_timing(False)
            gbs = ks["bytes_compulsory"] / (ks["ms_total"] * 1e-3) * 1e-9
            res[name] = {"us": 1e3 * ks["ms_total"] / ks["launches"], "GBs": round(gbs, 1),
                         "frac": round(gbs / peak, 4), "GFLOPS": round(ks["flops"] / (ks["ms_total"] * 1e-3) * 1e-9, 1)}
        for n in [int(v) for v in args.nrhs.split(",") if v]:
            ins = [ctx.new_field(prec) for _ in range(n)]
            outs = [ctx.new_field(prec) for _ in range(n)]
            for f in ins:
                ctx.spinor_load(f, prec, 0, psi)
            for _ in range(3):
                ctx.matpc_multi(outs, ins, prec)
            ctx.kernel_timing(True)
            for _ in range(max(5, args.reps // n)):
                ctx.matpc_multi(outs, ins, prec)
            ks = ctx.kernel_stats()
            ctx.kernel_timing(False)
            gbs = ks["bytes_compulsory"] / (ks["ms_total"] * 1e-3) * 1e-9
            res[f"matpc_x{n}"] = {"us_per_rhs": 1e3 * ks["ms_total"] / (ks["launches"] / 2) / n,
                                  "GFLOPS": round(ks["flops"] / (ks["ms_total"] * 1e-3) * 1e-9, 1),
                                  "GBs_multi_model": round(gbs, 1), "frac": round(gbs / peak, 4)}
        print(json.dumps(res), flush=True)
    ctx.close()


if __name__ == "__main__":
    main()
