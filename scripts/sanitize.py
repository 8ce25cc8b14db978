"""Small workloads for compute-sanitizer (racecheck / synccheck / memcheck) over the library's
hand-written synchronisation: the deterministic last-CTA reduction tails fused into the Dslash
epilogues and the BLAS kernels, the two-RHS-per-thread multi-RHS kernel with its per-RHS tails,
the kernel-initiated (P2P) halo's sequence flags in loopback, the NCCL-loopback split path, and
the batched solver.  8^4 lattice (a few CTAs per kernel keeps the tools' cost bounded).

    compute-sanitizer --tool racecheck python scripts/sanitize.py
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np  # noqa: E402

import qgen  # noqa: E402
from paper_1011_0024_b200 import qudax  # noqa: E402

DIMS = (8, 8, 8, 8)
K, CSW = 0.124, 1.0


def main():
    U = qgen.gauge(DIMS, 7001, eps=0.1)
    b = qgen.point_source(DIMS, 0, 0)
    srcs = [qgen.point_source(DIMS, s, c) for s, c in ((0, 0), (1, 1), (0, 2))]
    # fused-reduction Dslash (solver iterations), BLAS tails, device-side decisions, graphs
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, K, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
    _, st = ctx.solve(b, tol=1e-10, delta=1e-2, maxiter=200, prec=8, prec_sloppy=4)
    print("single solve", st["iters"], st["true_res"])
    # batched solver: two-RHS-per-thread kernel with per-RHS fused tails
    _, sts = ctx.solve_multi(srcs, tol=1e-10, delta=1e-2, maxiter=200, prec=8, prec_sloppy=4)
    print("batched", [s["iters"] for s in sts])
    ctx.close()
    # half precision sloppy (requantising stores + fused reductions)
    ctx = qudax.Context(DIMS)
    ctx.gauge_load(U, K, CSW, prec=8, recon=18, prec_sloppy=2, recon_sloppy=12)
    _, st = ctx.solve(b, tol=1e-10, delta=1e-2, maxiter=300, prec=8, prec_sloppy=2)
    print("double-half", st["iters"], st["true_res"])
    ctx.close()
    # kernel-initiated halo, loopback (pack -> own ghosts -> flags -> RANGE_TAIL Dslash)
    ctx = qudax.Context(DIMS, halo=qudax.HALO_P2P)
    ctx.gauge_load(U, K, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
    _, st = ctx.solve(b, tol=1e-10, delta=1e-2, maxiter=200, prec=8, prec_sloppy=4)
    print("p2p loopback", st["iters"], st["true_res"])
    ctx.close()
    # NCCL loopback split path (interior / boundary kernels, allreduce + coefficient kernel)
    ctx = qudax.Context(DIMS, comm=qudax.COMM_NCCL, nccl_id=qudax.nccl_unique_id())
    ctx.gauge_load(U, K, CSW, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
    _, st = ctx.solve(b, tol=1e-10, delta=1e-2, maxiter=200, prec=8, prec_sloppy=4)
    print("nccl loopback", st["iters"], st["true_res"])
    ctx.sync()
    print("sanitize workload done", flush=True)
    # leave without ncclCommDestroy: under compute-sanitizer NCCL's teardown did not return
    # (r02a: every tool had finished the workload, reported nothing, then hung in close)
    os._exit(0)


if __name__ == "__main__":
    main()
