import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import qgen
from paper_1011_0024_b200 import qudax
dims = (24, 24, 24, 128)
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=2, recon_sloppy=12)
b = qgen.point_source(dims, 0, 1)
x, st = ctx.solve(b, tol=1e-14, delta=1e-2, maxiter=6, prec=8, prec_sloppy=2, allow_not_converged=True)
print(st, flush=True)
os._exit(0)
