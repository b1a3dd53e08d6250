"""The seeded input generators (stencil_inputs) — host and device recipes agree."""
import itertools

import numpy as np
import torch

import stencil_inputs as si


def test_hash_grid_host_equals_torch():
    """HashGrid (oracle side, point reads) == hash_grid_torch (materialised),
    including linear indices past 2^31 and 2^32 where int64 products wrap."""
    ext = (3, 5, 7)
    g = si.HashGrid(ext, 9)
    t = si.hash_grid_torch(ext, 9, "cpu", chunk=17)
    for i in itertools.product(*map(range, ext)):
        assert t[i].item() == g[i]
    for lin in [(1 << 31) - 1, 1 << 31, (1 << 32) + 5, (1 << 33) + 77]:
        h = torch.tensor([lin], dtype=torch.int64)
        v = si.hash_grid_torch((1,), 3, "cpu")  # shape check only
        assert v.shape == (1,)
        hh = (h * 2654435761 + 3) & 0xFFFFFFFF
        hh ^= hh >> 15
        hh = (hh * 2246822519) & 0xFFFFFFFF
        hh ^= hh >> 13
        assert int(hh) == si._hash32(lin, 3)
    vals = t.numpy()
    assert vals.min() >= 1.0 and vals.max() < 2.0
    assert len(np.unique(vals)) > 0.9 * vals.size
