"""The seeded input generator: numpy and torch implementations agree bitwise,
values have the stated distribution and are exactly representable."""
import numpy as np
import pytest
import torch

import synth


@pytest.mark.parametrize("seed", [0, 1, 2, 3, 1002])
@pytest.mark.parametrize("start,count", [(0, 1000), (123457, 4099), ((1 << 32) - 7, 20), ((5 << 32) + 3, 9)])
@pytest.mark.parametrize("dist", ["sym", "pos"])
def test_numpy_torch_bitwise(seed, start, count, dist):
    a = synth.numpy_uniform(seed, start, count, dist)
    b = synth.torch_uniform(seed, start, count, dist, chunk=1000).numpy()
    assert a.dtype == np.float32 and b.dtype == np.float32
    assert np.array_equal(a.view(np.uint32), b.view(np.uint32))


def test_ranges_and_grid():
    v = synth.numpy_uniform(2, 0, 1 << 18, "sym")
    assert v.min() >= -1.0 and v.max() < 1.0
    assert np.all((v.astype(np.float64) * 2 ** 23) == np.round(v.astype(np.float64) * 2 ** 23))
    assert abs(float(v.mean())) < 0.01 and abs(float(v.var()) - 1 / 3) < 0.01
    p = synth.numpy_uniform(2, 0, 1 << 18, "pos")
    assert p.min() >= 0.0 and p.max() < 1.0 and abs(float(p.mean()) - 0.5) < 0.01


def test_rows_are_slices_of_the_full_matrix():
    full = synth.numpy_matrix_rows(2, 37, 0, 20)
    part = synth.numpy_matrix_rows(2, 37, 5, 11)
    assert np.array_equal(full[5:11], part)
    t = synth.torch_matrix_rows(2, 37, 5, 11).numpy()
    assert np.array_equal(t, part)


def test_seeds_differ():
    a = synth.numpy_uniform(0, 0, 64)
    b = synth.numpy_uniform(1, 0, 64)
    assert not np.array_equal(a, b)


def test_hadamard_orthogonal():
    H = synth.hadamard(32).astype(np.int64)
    assert np.array_equal(H.T @ H, 32 * np.eye(32, dtype=np.int64))
    assert np.all(H[0] == 1) and np.all(H[:, 0] == 1)


def test_numpy_wide_range_and_determinism():
    v = synth.numpy_wide(3, 0, 200_000)
    assert v.dtype == np.float32 and np.all(np.isfinite(v))
    assert np.array_equal(v, synth.numpy_wide(3, 0, 200_000))
    assert np.array_equal(v[1000:2000], synth.numpy_wide(3, 1000, 1000))  # counter-based: any slice
    a = np.abs(v[v != 0])
    assert a.max() < 2.0 ** 21 and a.max() > 2.0 ** 19
    assert np.mean(a < 2.0 ** -126) > 0.05  # subnormals present
    assert 0.45 < np.mean(v < 0) < 0.55
    # full significands: most values are not on the 2^-23-relative grid of U[-1,1)
    m = np.frexp(a[a >= 2.0 ** -126].astype(np.float64))[0]
    assert np.mean((m * 2 ** 24) % 2 != 0) > 0.4
