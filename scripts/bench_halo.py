"""Cost of the split (halo) Dslash path at N=1: Mhat through the unsplit kernel vs the NCCL
loopback (pack -> send/recv to self -> interior + boundary) vs the kernel-initiated P2P
loopback (pack stores into the ghosts + flag release -> interior + boundary acquire), and the
multi-dimensional split in loopback (Z, Z+T, Y+Z+T, all four: projected X/Y/Z faces, interior
box + boundary-list kernels).

    python scripts/bench_halo.py [--dims 32,32,32,64] [--reps 50] [--prec 4]
"""
import argparse
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import qgen  # noqa: E402
from paper_1011_0024_b200 import qudax  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--dims", default="32,32,32,64")
    ap.add_argument("--reps", type=int, default=50)
    ap.add_argument("--prec", type=int, default=4)
    ap.add_argument("--modes", default="", help="comma list of mode names to run (default all)")
    args = ap.parse_args()
    dims = tuple(int(v) for v in args.dims.split(","))
    U = qgen.gauge(dims, 1005, eps=0.1)
    psi = qgen.spinor(dims, 2005)
    res = {"dims": dims, "prec": args.prec}
    modes = (("unsplit", {}), ("nccl_loopback", {"comm": qudax.COMM_NCCL, "nccl_id": qudax.nccl_unique_id()}),
             ("p2p_loopback", {"halo": qudax.HALO_P2P}))
    nid = qudax.nccl_unique_id
    modes += tuple((f"nccl_loopback_split{m:04b}", {"comm": qudax.COMM_NCCL, "nccl_id": nid(), "split_mask": m})
                   for m in (0b0001, 0b0100, 0b1100, 0b1110, 0b1111))
    if args.modes:
        modes = tuple(m for m in modes if m[0] in args.modes.split(","))
    for name, kw in modes:
        ctx = qudax.Context(dims, **kw)
        ctx.gauge_load(U, 0.124, 1.0, prec=args.prec, recon=12 if args.prec != 8 else 18)
        a, b = ctx.new_field(args.prec), ctx.new_field(args.prec)
        ctx.spinor_load(a, args.prec, 0, psi)
        for _ in range(5):
            ctx.matpc(b, a, args.prec)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        ctx.sync()
        e0.record(ctx.stream)
        for _ in range(args.reps):
            ctx.matpc(b, a, args.prec)
        e1.record(ctx.stream)
        ctx.sync()
        res[name + "_matpc_us"] = round(1e3 * e0.elapsed_time(e1) / args.reps, 2)
        ctx.close()
    print(json.dumps(res), flush=True)


if __name__ == "__main__":
    main()
