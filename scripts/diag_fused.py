import os, sys, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import qgen
from paper_1011_0024_b200 import qudax
dims = (32, 32, 32, 64)
ctx = qudax.Context(dims)
ctx.gauge_load(qgen.gauge(dims, 1005, eps=0.1), 0.124, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
b = torch.from_numpy(qgen.spinor(dims, 2005).view(np.float64)).cuda()
out = {}
for prec in (4, 8):
    fi, fo = ctx.new_field(prec), ctx.new_field(prec)
    ctx.spinor_load_dev(fi, prec, 0, b)
    for _ in range(5):
        ctx.matpc(fo, fi, prec)
    ctx.kernel_timing(True)
    for _ in range(40):
        ctx.matpc(fo, fi, prec)
    ks = ctx.kernel_stats(prec=prec)
    ctx.kernel_timing(False)
    out[prec] = {"us_per_matpc": 1e3 * ks["ms_total"] / 40, "gflops": ks["flops"] / ks["ms_total"] * 1e-6}
print(os.environ.get("TAG", ""), json.dumps(out), flush=True)
os._exit(0)
