import os, sys
sys.path.insert(0, '/root/repo')
import numpy as np, torch, qgen
from paper_1011_0024_b200 import qudax
dims = (24, 24, 24, 128)
U = qgen.gauge(dims, 1003, eps=0.1)
ctx = qudax.Context(dims)
ctx.gauge_load(U, 0.124, 1.0, prec=8, recon=18, prec_sloppy=2, recon_sloppy=12, t_boundary=-1)
b = torch.from_numpy(qgen.point_source(dims, 0, 1).view(np.float64).reshape(-1)).cuda()
x = torch.zeros_like(b)
h = np.zeros(400)
st = ctx.solve_dev(x, b, tol=1e-14, delta=3e-3, maxiter=400, prec=8, prec_sloppy=2, allow_not_converged=True, history=h)
print(st)
print(" ".join("%.1e" % v for v in h[:400]))
