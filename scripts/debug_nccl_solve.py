"""Debug: NCCL-loopback solve variants (graphs on/off, poll_every, overlap) with progress output."""
import faulthandler
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
faulthandler.dump_traceback_later(50, exit=False)

import qgen  # noqa: E402
from paper_1011_0024_b200 import qudax  # noqa: E402

variant = sys.argv[1]
dims = (8, 8, 8, 16)
U = qgen.gauge(dims, 1003, eps=0.1)
b = qgen.point_source(dims, 1, 0)
flags = qudax.FLAG_DEBUG_SOLVER
if "nograph" in variant:
    flags |= qudax.FLAG_NO_GRAPHS
overlap = "noov" not in variant
poll = 1 if "poll1" in variant else 0
ctx = qudax.Context(dims, comm=qudax.COMM_NCCL, nccl_id=qudax.nccl_unique_id(), overlap=overlap, flags=flags)
print("ctx ok", flush=True)
ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
print("gauge ok", flush=True)
fi, fo = ctx.new_field(4), ctx.new_field(4)
ctx.spinor_load(fi, 4, 0, b)
ctx.matpc(fo, fi, 4)
ctx.sync()
print("matpc ok", ctx.norm2(fo, 4), flush=True)
t = time.time()
x, st = ctx.solve(b, tol=1e-10, delta=0.1, maxiter=30, prec=8, prec_sloppy=4, poll_every=poll,
                  allow_not_converged=True)
print("solve ok", st["iters"], st["true_res"], time.time() - t, flush=True)
ctx.close()
print("close ok", flush=True)
