import sys, os, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import qgen, oracle
from paper_1011_0024_b200 import qudax
DIMS=(8,8,8,16)
U=qgen.gauge(DIMS,1003,eps=0.1)
wc=oracle.WilsonClover(U,0.124,1.0,-1.0)
b=qgen.point_source(DIMS,0,0)
for mode in [(8,18,4,12,0.1,1e-12),(8,18,2,12,1e-2,1e-12),(8,18,2,12,1e-1,1e-12),(8,12,8,12,1e-5,1e-12),(4,12,2,12,0.1,1e-6),(8,18,8,18,0.0,1e-12)]:
    prec,recon,ps,rs,delta,tol=mode
    ctx=qudax.Context(DIMS)
    ctx.gauge_load(U,0.124,1.0,prec=prec,recon=recon,prec_sloppy=ps,recon_sloppy=rs)
    h=np.zeros(3000)
    x,st=ctx.solve(b,tol=tol,delta=delta,maxiter=3000,prec=prec,prec_sloppy=ps,allow_not_converged=True,history=h)
    res=np.linalg.norm(wc.M(x)-b)/np.linalg.norm(b)
    n=st['iters']
    print(mode, {k:st[k] for k in ('iters','reliable_updates','true_res','true_res_schur')}, 'oracle', res)
    print('  hist', np.array2string(h[:min(n,40)], precision=2), '...', h[max(0,n-5):n])
    ctx.close()
# oracle history for delta=0 check
bh=wc.prepare(b)
xe,hist=oracle.bicgstab(wc.matpc,bh,tol=1e-12,maxiter=3000)
print('oracle hist', np.array2string(np.array(hist[:40]),precision=2), len(hist))
