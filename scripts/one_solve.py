import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import qgen
from paper_1011_0024_b200 import qudax
dims = (32, 32, 32, 64)
ctx = qudax.Context(dims)
ctx.gauge_load(qgen.gauge(dims, 1005, eps=0.1), 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
b = torch.from_numpy(qgen.spinor(dims, 2005).view(np.float64)).cuda()
x = torch.zeros_like(b)
for it in (int(a) for a in sys.argv[1:] or ["20"]):
    st = ctx.solve_dev(x, b, tol=0.0, delta=float(os.environ.get("DELTA", "0")), maxiter=it, prec=4, prec_sloppy=4, allow_not_converged=True)
    print(st)
