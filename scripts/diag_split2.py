"""Debug: SS-variant vs plain kernel without ghosts (QUDAX_FORCE_SS), overlap on/off."""
import os, subprocess, sys
import numpy as np
sys.path.insert(0, ".")
import qgen
from paper_1011_0024_b200 import qudax

dims = (8, 4, 6, 8)
U = qgen.gauge(dims, 1221)
psi = qgen.spinor(dims, 1222)


def run(prec, **kw):
    c = qudax.Context(dims, **kw)
    c.gauge_load(U, 0.12, 1.0, prec=prec, recon=12)
    fi, fo = c.new_field(prec), c.new_field(prec)
    c.spinor_load(fi, prec, 1, psi)
    c.dslash(fo, fi, prec, 0, dagger=False, kind=0)
    c.sync()
    o = c.spinor_store(fo, prec, 0)
    c.close()
    return o


if len(sys.argv) > 1:
    np.save(sys.argv[1], run(2))
    sys.exit(0)
ref = run(2)
env = dict(os.environ, QUDAX_FORCE_SS="1")
subprocess.run([sys.executable, __file__, "/tmp/ss.npy"], env=env, check=True)
ss = np.load("/tmp/ss.npy")
d = np.abs(ref - ss).max(axis=(4, 5))
print("forced SS vs plain (no ghosts):", int((d > 0).sum()), "sites differ")
for ov in (True, False):
    lo = run(2, comm=qudax.COMM_NCCL, nccl_id=qudax.nccl_unique_id(), split_mask=2, overlap=ov)
    d = np.abs(ref - lo).max(axis=(4, 5))
    print("loop Y overlap", ov, int((d > 0).sum()), "sites differ", np.argwhere(d > 0)[:4].tolist())
