"""One mixed-precision solve through the N > 1 code path on one GPU (NCCL loopback: halo
send/recv to self and every global sum through ncclAllReduce on the one-rank communicator,
inside the cached solver graphs).  Run under ncu to list the kernels of the replayed graphs:

    ncu --metrics gpu__time_duration.sum --csv --log-file launches.csv python scripts/loopback_solve.py
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import qgen  # noqa: E402
from paper_1011_0024_b200 import qudax  # noqa: E402

dims = (16, 16, 16, 32)
U = qgen.gauge(dims, 1005, eps=0.1)
b = qgen.point_source(dims, 0, 0)
ctx = qudax.Context(dims, comm=qudax.COMM_NCCL, nccl_id=qudax.nccl_unique_id(), overlap=True)
ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
for _ in range(2):  # the second solve replays the cached batch graphs
    x, st = ctx.solve(b, tol=0.0, delta=1e-3, maxiter=12, prec=8, prec_sloppy=4, allow_not_converged=True)
    print("iters", st["iters"], "updates", st["reliable_updates"], "true_res", st["true_res"], flush=True)
ctx.close()
