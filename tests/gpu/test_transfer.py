"""Host <-> device copies of the host-buffer API (api.cpp h2d / d2h): pageable arrays larger
than the 8 MB direct-copy threshold go through the ring of pinned 32 MB chunks (several chunks
and a ragged tail here), pinned arrays straight through.  Both must move the bits exactly."""
import numpy as np
import pytest
import torch

import qgen
from paper_1011_0024_b200 import qudax

pytestmark = pytest.mark.gpu


def test_spinor_load_store_pageable_vs_device_path(torch_cuda):
    """spinor_load (pageable H2D through the ring) = spinor_load_dev of the same array moved by
    torch; spinor_store (H2D of the other parity + D2H through the ring) = spinor_store_dev
    moved back by torch — bit for bit."""
    dims = (16, 16, 16, 96)  # 72 MiB fp64 slab: two full 32 MiB chunks + a ragged tail
    psi = qgen.spinor(dims, 77)
    assert psi.nbytes > 2 * (32 << 20)
    psi_dev = torch.from_numpy(psi.view(np.float64).copy()).cuda()
    ctx = qudax.Context(dims)
    for p in range(2):
        a, b = ctx.new_field(8), ctx.new_field(8)
        ctx.spinor_load(a, 8, p, psi)
        ctx.spinor_load_dev(b, 8, p, psi_dev)
        ctx.sync()
        assert bool((a == b).all())
        host = np.zeros_like(psi)
        ctx.spinor_store(a, 8, p, out=host)
        dev = torch.zeros_like(psi_dev)
        ctx.spinor_store_dev(dev, a, 8, p)
        ctx.sync()
        got = host.view(np.float64).reshape(-1)
        ref = dev.cpu().numpy().reshape(-1)
        # spinor_store keeps the other parity's sites of `host` (zeros here), store_dev of `dev`
        assert np.array_equal(got, ref)
    ctx.close()


def test_solve_pageable_equals_pinned(torch_cuda):
    dims = (16, 16, 16, 48)  # 36 MiB slab: one full chunk + a ragged tail
    U = qgen.gauge(dims, 1402, eps=0.1)
    ctx = qudax.Context(dims)
    ctx.gauge_load(U, 0.12, 1.0, prec=8, recon=18, prec_sloppy=4, recon_sloppy=12)
    b = qgen.spinor(dims, 1403)
    x1, st1 = ctx.solve(b, tol=1e-9, delta=0.1, maxiter=2000, prec=8, prec_sloppy=4)
    bt = torch.from_numpy(b.view(np.float64).copy()).pin_memory()
    xt = torch.zeros_like(bt).pin_memory()
    x2, st2 = ctx.solve(bt, tol=1e-9, delta=0.1, maxiter=2000, prec=8, prec_sloppy=4, out=xt)
    assert st1["iters"] == st2["iters"]
    assert np.array_equal(x1.view(np.float64).reshape(-1), x2.numpy().reshape(-1))
    ctx.close()
