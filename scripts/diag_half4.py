import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import qgen
from paper_1011_0024_b200 import qudax
dims = (24, 24, 24, 128)
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
for Ps, R, delta in ((2, 12, 1e-2), (2, 12, 0.1), (4, 12, 0.1)):
    ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=Ps, recon_sloppy=R)
    res = []
    for colour in range(3):
        for spin in range(2):
            b = qgen.point_source(dims, spin, colour)
            x, st = ctx.solve(b, tol=1e-14, delta=delta, maxiter=1500, prec=8, prec_sloppy=Ps, allow_not_converged=True)
            res.append((st["iters"], st["reliable_updates"], st["restarts"], "%.1e" % st["true_res"], "%.3f" % st["secs"]))
    print(Ps, R, delta, res, flush=True)
os._exit(0)
