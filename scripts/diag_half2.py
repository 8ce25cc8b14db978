import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import qgen
from paper_1011_0024_b200 import qudax
dims = (24, 24, 24, 128)
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
for Ps, delta in ((2, 1e-2),):
    ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=Ps, recon_sloppy=12)
    for colour in range(3):
        for spin in range(2):
            b = qgen.point_source(dims, spin, colour)
            h = np.zeros(3000)
            x, st = ctx.solve(b, tol=1e-14, delta=delta, maxiter=1500, prec=8, prec_sloppy=Ps, allow_not_converged=True, history=h)
            n = st["iters"]
            print(colour, spin, {k: st[k] for k in ("iters", "reliable_updates", "true_res")}, flush=True)
            print("   ", np.array2string(h[:n:25][:30], precision=1), flush=True)
os._exit(0)
