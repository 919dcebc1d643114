"""Pins for the CPU oracle -- none of them re-types the
oracle's formula: each checks it against a closed form, an independent
formulation (banded Toeplitz matrices), an independent library routine
(torch conv2d in float64), an invariance, or a hand-derived worked example.

Runs on CPU only (-m "not gpu")."""
import os

import numpy as np
import pytest

import oracle
from paper_conf_asplos_phothilimthanaara13_b200 import synth
from tests.parity import rel_error

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")


def _rand(h, w, seed):
    return synth.uniform_image(h, w, seed)


# ---- P1: delta kernel -> exact shifted crop (correlation, anchor, valid shape)
@pytest.mark.parametrize("K", [1, 2, 3, 4, 5, 8, 17])
def test_delta_kernel_exact(K):
    img = _rand(23, 31, 11)          # H != W catches an axis swap
    ho, wo = 23 - K + 1, 31 - K + 1
    for m in range(K):
        k = synth.delta_kernel(K, m)
        want = img[m:m + ho, m:m + wo].astype(np.float64)
        assert np.array_equal(oracle.convolve2d(img, k), want)
        assert np.array_equal(oracle.separable(img, k), want)
        assert np.array_equal(oracle.convolve_rows(img, k), img[:, m:m + wo])
        buf = np.arange(23 * 7, dtype=np.float64).reshape(23, 7)
        assert np.array_equal(oracle.convolve_columns(buf, k), buf[m:m + ho])


# ---- P2: constant image x box kernel
@pytest.mark.parametrize("K", [1, 3, 6, 17])
def test_constant_box_closed_form(K):
    a = 7.0
    img = np.full((20, 19), a, np.float32)
    out = oracle.convolve2d(img, synth.box_kernel(K))
    assert out.shape == (20 - K + 1, 19 - K + 1)
    assert np.all(out == a * K * K)
    kn = synth.box_kernel(K, normalized=True)          # k_i = fl32(1/K)
    out_n = oracle.separable(img, kn)
    closed = a * (K * float(kn[0])) ** 2                # = a up to fl32(1/K) rounding
    assert np.allclose(out_n, closed, rtol=1e-14, atol=0)
    assert abs(closed - a) <= a * 3 * 2.0 ** -24


# ---- P3: linearity and power-of-two scaling (quadratic role of k)
def test_linearity_and_scaling():
    # 12-bit inputs so that alpha*x + beta*y below is exact in float32
    x = (np.floor(_rand(30, 27, 1) * 4096) / 4096).astype(np.float32)
    y = (np.floor(_rand(30, 27, 2) * 4096) / 4096).astype(np.float32)
    k = synth.random_kernel(7, 3, signed=True)
    cx, sx = oracle.convolve2d(x, k, with_absum=True)
    cy, sy = oracle.convolve2d(y, k, with_absum=True)
    alpha, beta = np.float32(0.75), np.float32(-1.5)
    z = (alpha * x + beta * y).astype(np.float32)
    assert np.array_equal(z.astype(np.float64), 0.75 * x.astype(np.float64) - 1.5 * y)
    cz = oracle.convolve2d(z, k)
    scale = abs(alpha) * sx + abs(beta) * sy
    assert np.max(np.abs(cz - (alpha * cx + beta * cy)) / scale) < 1e-14
    for p in (-3, 2, 5):
        assert np.array_equal(oracle.convolve2d((x * 2.0 ** p).astype(np.float32), k), cx * 2.0 ** p)
        assert np.array_equal(oracle.convolve2d(x, (k * 2.0 ** p).astype(np.float32)), cx * 4.0 ** p)


# ---- P4: separable == 2D == banded-Toeplitz matrix form A . In . B^T (brute force)
def _toeplitz(n_out, n_in, k):
    a = np.zeros((n_out, n_in))
    for r in range(n_out):
        a[r, r:r + k.size] = k
    return a


def test_separable_equals_2d_equals_matrix_form_bruteforce():
    rng = np.random.default_rng(5)
    for h in range(1, 10):
        for w in range(1, 10):
            img = rng.uniform(-1, 1, (h, w)).astype(np.float32)
            for K in range(1, min(h, w) + 1):
                k = rng.uniform(-1, 1, K).astype(np.float32)
                kd = k.astype(np.float64)
                mat = _toeplitz(h - K + 1, h, kd) @ img.astype(np.float64) @ _toeplitz(w - K + 1, w, kd).T
                c2, s = oracle.convolve2d(img, k, with_absum=True)
                sep = oracle.separable(img, k)
                assert c2.shape == mat.shape == sep.shape
                assert np.max(np.abs(c2 - mat) / s) < 1e-13
                assert np.max(np.abs(sep - mat) / s) < 1e-13


# ---- P4b: integer-exact data -> every formulation agrees exactly
def test_integer_exact_all_forms_agree():
    img = synth.integer_image(21, 26, 9)
    for K in (1, 2, 5, 9, 17):
        k = synth.integer_kernel(K, K)
        kd = k.astype(np.float64)
        mat = _toeplitz(21 - K + 1, 21, kd) @ img.astype(np.float64) @ _toeplitz(26 - K + 1, 26, kd).T
        assert np.array_equal(oracle.convolve2d(img, k), mat)
        assert np.array_equal(oracle.separable(img, k), mat)
        assert np.max(np.abs(mat)) <= 17 * 17 * 9 * 15


# ---- ramp closed form: In = a r + b c + g  ->  Out = S^2 In(r,c) + S M (a + b)
@pytest.mark.parametrize("K", [1, 2, 3, 4, 7, 16, 17])
def test_ramp_closed_form_orientation(K):
    h, w, a, b, g = 29, 33, 3.0, -2.0, 5.0
    r = np.arange(h)[:, None]
    c = np.arange(w)[None, :]
    img = (a * r + b * c + g).astype(np.float32)
    k = np.arange(1, K + 1, dtype=np.float32) * np.float32(1 if K % 2 else -1)   # asymmetric
    S = float(k.sum())
    M = float((np.arange(K) * k).sum())
    ro, co = np.arange(h - K + 1)[:, None], np.arange(w - K + 1)[None, :]
    want = S * S * (a * ro + b * co + g) + S * M * (a + b)
    assert np.array_equal(oracle.convolve2d(img, k), want)
    assert np.array_equal(oracle.separable(img, k), want)


# ---- worked example fixture (hand-derived, tests/golden/ramp_4x5_k3.txt)
def _read_golden(name):
    lines = [ln.strip() for ln in open(os.path.join(GOLDEN, name)) if ln.strip() and not ln.startswith("#")]
    it = iter(lines)
    meta, inp, out = {}, [], []
    section = None
    for ln in it:
        if ln in ("input", "output"):
            section = ln
            continue
        if section == "input":
            inp.append([float(v) for v in ln.split()])
        elif section == "output":
            out.append([float(v) for v in ln.split()])
        else:
            key, *vals = ln.split()
            meta[key] = vals
    return meta, np.array(inp, np.float32), np.array(out, np.float64)


def test_golden_worked_example():
    meta, img, want = _read_golden("ramp_4x5_k3.txt")
    k = np.array([float(v) for v in meta["kernel"]], np.float32)
    assert img.shape == (int(meta["h"][0]), int(meta["w"][0]))
    assert np.array_equal(oracle.convolve2d(img, k), want)
    assert np.array_equal(oracle.separable(img, k), want)


# ---- P6: independent library routine (torch conv2d is cross-correlation, valid padding)
def test_torch_conv2d_float64_agrees():
    torch = pytest.importorskip("torch")
    for K, seed in ((3, 1), (8, 2), (17, 3)):
        img = _rand(61, 47, seed)
        k = synth.random_kernel(K, seed, signed=True)
        ref = torch.nn.functional.conv2d(
            torch.from_numpy(img).double()[None, None],
            torch.outer(torch.from_numpy(k).double(), torch.from_numpy(k).double())[None, None])[0, 0].numpy()
        out, s = oracle.convolve2d(img, k, with_absum=True)
        assert np.max(np.abs(out - ref) / s) < 1e-12


# ---- P7: invariances
def test_transpose_translation_and_k1():
    img = _rand(40, 35, 4)
    k = synth.random_kernel(9, 4, signed=True)
    out, s = oracle.convolve2d(img, k, with_absum=True)
    out_t = oracle.convolve2d(np.ascontiguousarray(img.T), k)
    assert np.max(np.abs(out_t - out.T) / s.T) < 1e-15
    dr, dc = 5, 3
    crop = oracle.convolve2d(np.ascontiguousarray(img[dr:, dc:]), k)
    assert np.max(np.abs(crop - out[dr:, dc:]) / s[dr:, dc:]) < 1e-15
    k1 = np.array([0.5], np.float32)
    assert np.array_equal(oracle.convolve2d(img, k1), img.astype(np.float64) * 0.25)


def test_absum_is_output_for_nonnegative_data():
    img = _rand(33, 30, 6)
    out, s = oracle.convolve2d(img, synth.binomial_kernel(11), with_absum=True)
    assert np.array_equal(out, s)
    out2, s2 = oracle.convolve2d(img - np.float32(0.5), synth.random_kernel(5, 1, signed=True), with_absum=True)
    assert np.all(s2 >= np.abs(out2))


# ---- P8: float32 evaluation in the kernels' fixed order stays inside the tolerance.
# Emulates the row-partial order (R6) with numpy float32 (separate
# multiply and add: two roundings per term, a looser bound than fma).
def test_float32_fixed_order_error_bound():
    img = _rand(64, 64, 8)
    for K in (3, 9, 17):
        k = synth.binomial_kernel(K)
        o, s = oracle.convolve2d(img, k, with_absum=True)
        ho, wo = 64 - K + 1, 64 - K + 1
        acc = np.zeros((ho, wo), np.float32)
        for j in range(K):
            part = np.zeros((ho, wo), np.float32)
            for i in range(K):
                part = part + np.float32(k[i] * k[j]) * img[j:j + ho, i:i + wo]
            acc = acc + part
        err = rel_error(acc, o, s)
        assert err <= (2 * K + 2) * 2.0 ** -24
        assert err < 1e-5


# ---- P9: band decomposition == whole image (partition + one-sided halo)
@pytest.mark.parametrize("G", [1, 2, 3, 4, 8])
def test_band_decomposition_exact(G):
    img = _rand(77, 41, 10)
    for K in (1, 3, 8):
        k = synth.random_kernel(K, K)
        assert np.array_equal(oracle.convolve2d_bands(img, k, G), oracle.convolve2d(img, k))


def test_band_rows_cover_output():
    for ho in (1, 7, 16368):
        for G in (1, 2, 3, 8):
            edges = [oracle.band_rows(ho, G, g) for g in range(G)]
            assert edges[0][0] == 0 and edges[-1][1] == ho
            assert all(edges[g][1] == edges[g + 1][0] for g in range(G - 1))
            sizes = [b - a for a, b in edges]
            assert max(sizes) - min(sizes) <= 1


def test_threads_do_not_change_result():
    img = _rand(50, 44, 12)
    k = synth.random_kernel(6, 2, signed=True)
    a = oracle.convolve2d(img, k, nthreads=1)
    b = oracle.convolve2d(img, k, nthreads=7)
    assert np.array_equal(a, b)


def test_rejects_bad_shapes():
    with pytest.raises(ValueError):
        oracle.convolve2d(np.zeros((3, 3), np.float32), np.ones(4, np.float32))
    with pytest.raises(TypeError):
        oracle.convolve2d(np.zeros((5, 5), np.float64), np.ones(3, np.float32))


def test_synth_is_counter_based():
    full = synth.uniform_image(40, 33, 77)
    band = synth.uniform_image(40, 33, 77, rows=(13, 29))
    assert np.array_equal(full[13:29], band)
    assert full.min() >= 0 and full.max() < 1
    assert np.all(full * 2 ** 24 == np.floor(full * 2 ** 24))
    k = synth.binomial_kernel(17)
    assert k.sum() == 1.0 and k[8] == 12870 / 2 ** 16
