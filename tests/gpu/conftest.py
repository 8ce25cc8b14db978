import numpy as np
import pytest


def rel_l2(a, b):
    return float(np.linalg.norm((a - b).ravel()) / np.linalg.norm(b.ravel()))


TOL = {8: 1e-12, 4: 1e-5, 2: 5e-3}  # BASELINE.json north_star: fp64 / fp32 / half relative L2


@pytest.fixture(scope="session")
def torch_cuda():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    return torch
