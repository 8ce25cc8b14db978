"""Batched vs independent double-half solves of the config-3 sources: iterations per system
(run with and without QUDAX_MR_OFF to localise a difference)."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import qgen
from paper_1011_0024_b200 import qudax
dims = (24, 24, 24, 128)
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
srcs = [qgen.point_source(dims, s, c) for c in range(3) for s in range(2)]
for ps, delta in ((2, 1e-2), (4, 1e-3)):
    ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=ps, recon_sloppy=12, t_boundary=-1)
    h = np.zeros(400)
    _, sts = ctx.solve_multi(srcs, tol=1e-14, delta=delta, maxiter=4000, prec=8, prec_sloppy=ps, history=h)
    h1 = np.zeros(400)
    ind0 = ctx.solve(srcs[0], tol=1e-14, delta=delta, maxiter=4000, prec=8, prec_sloppy=ps, history=h1)[1]
    first = next((k for k in range(400) if h[k] != h1[k]), None)
    print("sloppy", ps, "batched iters", [s["iters"] for s in sts], "independent sys0", ind0["iters"],
          "first differing history entry", first, h[first] if first is not None else None, h1[first] if first is not None else None, flush=True)
ctx.close()
