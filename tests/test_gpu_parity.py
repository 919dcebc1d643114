"""GPU parity: the CUDA path through the C ABI vs the CPU oracle, element by element.

Bar (tests/parity.py): max |g - o| / S <= 1e-5 with S = sum |k_i k_j In| (= plain
relative error for the non-negative benchmark data); bit-exact for integer-valued
data, delta kernels and shape/halo handling; canaries around every output buffer
must be untouched.  Runs only on a B200 (-m gpu)."""
import numpy as np
import pytest

import oracle
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc
from paper_conf_asplos_phothilimthanaara13_b200 import synth
from tests.parity import TOL, rel_error

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

CANDS = [
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 0),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 1),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 2),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 3),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 4),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 5),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 0, 1),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_DIRECT, 1),
    sc.Choice(sc.SEPCONV_2D, sc.MAP_TMA, 0),
    sc.Choice(sc.SEPCONV_2D, sc.MAP_DIRECT, 0),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 0),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_DIRECT, 0),
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 1, 2),   # store path 2 (two 8-byte stores per lane)
    sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 4, 2),
]
IDS = [c.name for c in CANDS]
GUARD = 4096          # floats of NaN canary on each side of every output buffer


def run_gpu(img, k, choice=None, variant=None, ld_in=0, ld_out=0, off_in=0, off_out=0, plan=None):
    """Run one convolution through the C ABI with canary-guarded buffers; return out [n][ho][wo]."""
    x = np.asarray(img, np.float32)
    if x.ndim == 2:
        x = x[None]
    n, h, w = x.shape
    K = int(np.asarray(k).size)
    ho, wo = h - K + 1, w - K + 1
    ld_in = ld_in or w
    ld_out = ld_out or wo
    src = np.full((n, h, ld_in), np.nan, np.float32)
    src[:, :, :w] = x
    dev_in = torch.empty(off_in + n * h * ld_in + 64, dtype=torch.float32, device="cuda")
    dev_in[off_in:off_in + src.size] = torch.from_numpy(src.reshape(-1)).cuda()
    out_len = n * ho * ld_out
    dev_out = torch.full((2 * GUARD + off_out + out_len,), float("nan"), dtype=torch.float32, device="cuda")
    p = plan or sc.Plan(h, w, K, n=n, ld_in=ld_in, ld_out=ld_out)
    pin = dev_in.data_ptr() + 4 * off_in
    pout = dev_out.data_ptr() + 4 * (GUARD + off_out)
    if choice is not None:
        p.run_choice(pin, k, pout, choice)
    else:
        p.run(pin, k, pout, variant or "auto")
    torch.cuda.synchronize()
    full = dev_out.cpu().numpy()
    assert np.all(np.isnan(full[:GUARD + off_out])), "canary before the output was overwritten"
    assert np.all(np.isnan(full[GUARD + off_out + out_len:])), "canary after the output was overwritten"
    body = full[GUARD + off_out:GUARD + off_out + out_len].reshape(n, ho, ld_out)
    if ld_out > wo:
        assert np.all(np.isnan(body[:, :, wo:])), "pitch padding of the output was written"
    out = body[:, :, :wo]
    assert not np.any(np.isnan(out)), "an output cell was not written"
    return out


def check(img, k, out):
    o, s = oracle.convolve2d(img, k, with_absum=True)
    err = rel_error(out, o, s)
    assert err <= TOL, f"max relative error {err:.3e} > {TOL}"
    return err


@pytest.mark.parametrize("choice", CANDS, ids=IDS)
@pytest.mark.parametrize("shape", [(67, 131), (300, 1100)])
def test_random_all_widths(choice, shape):
    h, w = shape
    img = synth.uniform_image(h, w, seed=100 + h) - np.float32(0.5)
    for K in range(1, 18):
        k = synth.random_kernel(K, seed=K, signed=True)
        out = run_gpu(img, k, choice)[0]
        check(img, k, out)


@pytest.mark.parametrize("choice", CANDS, ids=IDS)
def test_integer_exact_bitwise(choice):
    img = synth.integer_image(150, 1030, seed=7)
    for K in (1, 2, 3, 8, 16, 17):
        k = synth.integer_kernel(K, seed=K)
        out = run_gpu(img, k, choice)[0]
        want = oracle.convolve2d(img, k).astype(np.float32)
        assert np.array_equal(out, want), f"K={K}"


@pytest.mark.parametrize("choice", CANDS, ids=IDS)
def test_delta_kernel_bitwise(choice):
    img = synth.uniform_image(90, 260, seed=3)
    for K in (5, 17):
        for m in (0, K // 2, K - 1):
            out = run_gpu(img, synth.delta_kernel(K, m), choice)[0]
            assert np.array_equal(out, img[m:m + 90 - K + 1, m:m + 260 - K + 1])


def test_fused_equals_unfused_and_mappings_agree_bitwise():
    img = synth.uniform_image(333, 2100, seed=11)
    for K in (3, 8, 17):
        k = synth.random_kernel(K, seed=K, signed=True)
        outs = [run_gpu(img, k, c)[0] for c in CANDS]
        sep = [o for o, c in zip(outs, CANDS) if c.algo == sc.SEPCONV_SEPARABLE]
        two = [o for o, c in zip(outs, CANDS) if c.algo == sc.SEPCONV_2D]
        for o in sep[1:]:
            assert np.array_equal(o, sep[0])
        for o in two[1:]:
            assert np.array_equal(o, two[0])


@pytest.mark.parametrize("choice", CANDS, ids=IDS)
def test_pitched_and_misaligned(choice):
    img = synth.uniform_image(120, 517, seed=5)
    for K, ld_in, ld_out, off_in, off_out in ((3, 520, 515, 0, 0), (7, 517, 511, 1, 1), (16, 523, 505, 3, 2),
                                               (17, 528, 512, 0, 3)):
        k = synth.random_kernel(K, seed=K)
        out = run_gpu(img, k, choice, ld_in=ld_in, ld_out=ld_out, off_in=off_in, off_out=off_out)[0]
        check(img, k, out)


@pytest.mark.parametrize("choice", CANDS, ids=IDS)
def test_batch_equals_single_images(choice):
    imgs = np.stack([synth.uniform_image(70, 300, seed=50, n=i) for i in range(3)])
    K = 9
    k = synth.binomial_kernel(K)
    batch = run_gpu(imgs, k, choice)
    for i in range(3):
        assert np.array_equal(batch[i], run_gpu(imgs[i], k, choice)[0])
        check(imgs[i], k, batch[i])


@pytest.mark.parametrize("choice", CANDS, ids=IDS)
def test_degenerate_shapes(choice):
    for h, w, K in ((17, 17, 17), (1, 1, 1), (5, 300, 5), (300, 5, 5), (64, 64, 3), (2, 9000, 2)):
        img = synth.uniform_image(h, w, seed=h * w)
        k = synth.random_kernel(K, seed=1)
        out = run_gpu(img, k, choice)[0]
        assert out.shape == (h - K + 1, w - K + 1)
        check(img, k, out)


def test_variants_and_auto_default():
    img = synth.uniform_image(64, 64, seed=0x5EC0000)       # BASELINE config C1
    k = synth.binomial_kernel(3)
    for v in ("2d", "separable", "auto"):
        check(img, k, run_gpu(img, k, variant=v)[0])


@pytest.mark.parametrize("cfg", range(6))
@pytest.mark.parametrize("store_path", [0, 1, 2])
def test_right_edge_store_paths(cfg, store_path):
    """Right-edge warps on the 8-byte store paths (store mode 3: fused TMA kernels, K >= 13,
    widths <= 8192, even output widths): output widths = 2 and 0 mod 4, rows
    8- and 16-byte aligned (a pitched output shifts every row start by 8 bytes), strips that end
    inside a warp, next to the odd widths that keep the general store path -- every cell against
    the oracle, canaries around every output."""
    c = sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, store_path)
    for w in (130, 642, 2048, 2051, 3520):
        img = synth.uniform_image(40, w, seed=w) - np.float32(0.5)
        for K in (13, 14, 15, 17):
            k = synth.random_kernel(K, seed=K + w, signed=True)
            wo = w - K + 1
            for ld_out in (0, wo + 2, wo + 1):
                out = run_gpu(img, k, c, ld_out=ld_out)[0]
                check(img, k, out)


def test_set_choice_drives_auto():
    """sepconv_set_choice: AUTO resolves to the set candidate (bitwise the output run_choice gives
    for it, within the bound of the oracle), the other variants keep their resolution, and a
    choice of the wrong algorithm for a variant is rejected."""
    h, w, K = 300, 1100, 7
    img = synth.uniform_image(h, w, seed=77)
    k = synth.binomial_kernel(K)
    p = sc.Plan(h, w, K)
    sep_before = p.get_choice("separable")
    for cfg in (3, 5):
        c = sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg)
        p.set_choice(c)
        got = p.get_choice("auto")
        assert got.key() == c.key() and got.source == sc.SRC_EXPLICIT
        assert p.get_choice("separable").key() == sep_before.key()
        via_auto = run_gpu(img, k, variant="auto", plan=p)[0]
        via_choice = run_gpu(img, k, c, plan=p)[0]
        assert np.array_equal(via_auto, via_choice)
        check(img, k, via_auto)
    with pytest.raises(sc.SepconvError) as ei:
        p.set_choice(sc.Choice(sc.SEPCONV_2D, sc.MAP_TMA, 0), "separable")
    assert ei.value.code == "E_INVALID"


def test_tune_choice_is_valid_and_cached(tmp_path):
    cache = str(tmp_path / "tune.jsonl")
    img = synth.uniform_image(512, 768, seed=9)
    k = synth.binomial_kernel(11)
    p = sc.Plan(512, 768, 11)
    best = p.tune(reps=3, cache_path=cache, force=True)
    assert best.median_us > 0
    names = {c.name for c in p.candidates()}
    assert best.base_name in names and best.source == sc.SRC_TUNED
    for v in ("2d", "separable", "auto"):
        c = p.get_choice(v)
        assert c.median_us > 0
        assert c.base_name in names
    # ties within 1% go to fewer passes / the lower candidate index (R17)
    assert p.get_choice("auto").median_us <= min(p.get_choice("2d").median_us, p.get_choice("separable").median_us) * 1.01
    check(img, k, run_gpu(img, k, variant="auto", plan=p)[0])
    q = sc.Plan(512, 768, 11)
    again = q.tune(reps=3, cache_path=cache)                 # cache hit: no re-measurement
    assert again == best


def test_run_host_pipeline():
    h, w, K = 2500, 16384, 5                                 # 10 row bands of 256 rows (16 MB chunks)
    img = synth.uniform_image(h, w, seed=21)
    k = synth.binomial_kernel(K)
    src = torch.from_numpy(img).pin_memory()
    dst = torch.empty((h - K + 1, w - K + 1), dtype=torch.float32).pin_memory()
    p = sc.Plan(h, w, K)
    for v in ("separable", "2d"):
        dst.fill_(float("nan"))
        p.run_host(src, k, dst, v)
        check(img, k, dst.numpy())


def test_batch_with_narrow_edge_strip_every_fused_config():
    """A batch whose images end in a one-warp CTA strip (16400 columns: 16 full 1024-column
    strips + 8 columns) under the window schedule: CTAs take segments of different strips, so
    the lockstep configurations must not mix barrier counts between segments (a hang/trap
    before the per-segment CTA barrier).  Every fused TMA configuration, both store paths."""
    n, h, w, K = 2, 700, 16400, 9       # 692 output rows: q = 4 windows + 12 CTAs x 3 short segments
    imgs = np.stack([synth.uniform_image(h, w, seed=91, n=i) for i in range(n)])
    k = synth.binomial_kernel(K)
    outs = [run_gpu(imgs, k, c) for c in CANDS if c.algo == sc.SEPCONV_SEPARABLE and c.fused]
    for o in outs[1:]:
        assert np.array_equal(o, outs[0])
    for i in range(n):
        check(imgs[i], k, outs[0][i])


def test_run_host_batch_and_pitch_equal_device_run():
    """Host pipeline over a batch (bands restart at every image: no halo carry across images)
    with pitched buffers: bitwise equal to the device-resident run of the same plan."""
    n, h, w, K = 2, 700, 16400, 9                          # 16 MB bands of 255 rows: 3 per image
    imgs = np.stack([synth.uniform_image(h, w, seed=77, n=i) for i in range(n)])
    ld_in, ld_out = w + 12, w - K + 1 + 5
    src = np.zeros((n, h, ld_in), np.float32)
    src[:, :, :w] = imgs
    src_t = torch.from_numpy(src).pin_memory()
    dst_t = torch.full((n, h - K + 1, ld_out), float("nan")).pin_memory()
    k = synth.random_kernel(K, seed=3, signed=True)
    p = sc.Plan(h, w, K, n=n, ld_in=ld_in, ld_out=ld_out)
    p.run_host(src_t, k, dst_t, "separable")
    dev_out = torch.full((n, h - K + 1, ld_out), float("nan"), device="cuda")
    p.run(src_t.cuda(), k, dev_out, "separable")
    torch.cuda.synchronize()
    got = dst_t.numpy()
    assert np.array_equal(got[:, :, :w - K + 1], dev_out.cpu().numpy()[:, :, :w - K + 1])
    assert np.all(np.isnan(got[:, :, w - K + 1:]))                 # pitch padding untouched
    for i in range(n):
        check(imgs[i], k, got[i, :, :w - K + 1])


def test_errors():
    p = sc.Plan(64, 64, 3)
    buf = torch.zeros(64 * 64 * 2, device="cuda")
    k = synth.binomial_kernel(3)
    with pytest.raises(sc.SepconvError) as ei:
        p.run(buf.data_ptr(), k, buf.data_ptr() + 4 * 100, "auto")
    assert ei.value.code == "E_ALIAS"
    with pytest.raises(sc.SepconvError) as ei:
        p.run(buf.data_ptr() + 2, k, buf.data_ptr() + 4 * 5000, "auto")
    assert ei.value.code == "E_ALIGN"
    with pytest.raises(sc.SepconvError) as ei:
        sc.lib()
        st = sc.lib().sepconv_run(p.handle, buf.data_ptr(), None, buf.data_ptr() + 4 * 5000, 2, 0)
        sc._check(st, "sepconv_run")
    assert ei.value.code == "E_INVALID"
    with pytest.raises(sc.SepconvError) as ei:
        p.run(buf.data_ptr(), k, buf.data_ptr() + 4 * 5000, 7)
    assert ei.value.code == "E_INVALID"


def test_launch_count_increases():
    before = sc.launch_count()
    img = synth.uniform_image(64, 300, seed=1)
    run_gpu(img, synth.binomial_kernel(5), CANDS[10])          # unfused: 2 launches
    assert sc.launch_count() == before + 2


# ---- full BASELINE size, untuned plan (static default and 2D), sampled rows -----------------
@pytest.mark.parametrize("K", [3, 5, 7, 9, 11, 13, 15, 17])
def test_full_size_16384_sampled_rows(K, _big_image):
    """The untuned plan at 16384^2 (AUTO = the static default, and 2D) on sampled rows plus the
    [0, 1) range property; the tuned configurations bench.py times are compared with the
    oracle on every output cell in tests/test_gpu_fullsize.py."""
    img, dev_in = _big_image
    H = W = 16384
    ho, wo = H - K + 1, W - K + 1
    k = synth.binomial_kernel(K)
    p = sc.Plan(H, W, K)
    out = torch.empty((ho, wo), dtype=torch.float32, device="cuda")
    rows = sorted({0, 1, 1023, 1024, 8191, ho // 2, ho - 2, ho - 1})
    for v in ("auto", "2d"):
        out.fill_(float("nan"))
        p.run(dev_in, k, out, v)
        torch.cuda.synchronize()
        assert not torch.isnan(out).any().item()
        got = out[rows].cpu().numpy()
        for i, r in enumerate(rows):
            o, s = oracle.convolve2d(np.ascontiguousarray(img[r:r + K]), k, with_absum=True)
            assert rel_error(got[i:i + 1], o, s) <= TOL, (v, r)
        # property at full size: non-negative data and kernel summing to 1 keep every output in [0, 1)
        assert float(out.min()) >= 0.0 and float(out.max()) < 1.0


@pytest.fixture(scope="module")
def _big_image():
    img = synth.uniform_image(16384, 16384, seed=synth.BENCH_SEED_BASE + 3)
    dev = torch.from_numpy(img).cuda()
    yield img, dev
    del dev


# ---- row bands on one GPU: partition + interior/tail split of sepconv_run_band ---------------
@pytest.mark.parametrize("G,K", [(2, 3), (3, 9), (4, 17), (3, 1)])
def test_run_band_external_halo_equals_whole_image(G, K):
    """Each band runs through sepconv_run_band (interior rows, then the K-1 tail rows after
    the halo event) with the halo rows copied in by the test instead of NCCL (external-halo
    mode); the concatenated bands must equal the single-GPU output bit for bit."""
    H, W = 1000, 2100
    img = synth.uniform_image(H, W, seed=31)
    k = synth.random_kernel(K, seed=K, signed=True)
    full_plan = sc.Plan(H, W, K)
    dev = torch.from_numpy(img).cuda()
    want = torch.empty((H - K + 1, W - K + 1), device="cuda")
    for v in ("separable", "2d"):
        full_plan.run(dev, k, want, v)
        parts = []
        for g in range(G):
            r0, rows, owned, alloc = sc.band(H, K, G, g)
            band = torch.full((alloc, W), float("nan"), device="cuda")
            band[:owned] = dev[r0:r0 + owned]
            if g < G - 1:                     # the transport's job: K-1 rows of band g+1
                band[owned:alloc] = dev[r0 + owned:r0 + alloc]
            p = sc.Plan(alloc, W, K)
            p.comm_init(None, G, g)
            out = torch.full((rows, W - K + 1), float("nan"), device="cuda")
            p.run_band(band, k, out, v)
            parts.append(out)
        torch.cuda.synchronize()
        got = torch.cat(parts, 0)
        assert torch.equal(got, want), v


def test_repeated_calls_refresh_weights_and_choices():
    """sepconv_run's replay fast path (same plan and pointers) must still take each call's
    weights, candidate and schedule: alternate kernels, fused configurations and schedule
    overrides on the same buffers, every result checked against the oracle or bitwise."""
    h, w, K = 700, 1500, 9
    img = synth.uniform_image(h, w, seed=17)
    dev = torch.from_numpy(img).cuda()
    out = torch.empty((h - K + 1, w - K + 1), device="cuda")
    p = sc.Plan(h, w, K)
    ka, kb = synth.random_kernel(K, seed=1, signed=True), synth.random_kernel(K, seed=2, signed=True)
    for k in (ka, kb, ka):
        out.fill_(float("nan"))
        p.run(dev, k, out, "separable")
        torch.cuda.synchronize()
        check(img, k, out.cpu().numpy())
    ref = out.clone()
    for cfg in range(6):
        for parts in (0, 3):
            out.fill_(float("nan"))
            p.run_choice(dev, ka, out, sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, sched_parts=parts))
            torch.cuda.synchronize()
            assert torch.equal(out, ref), (cfg, parts)
    run = p.bind(dev, kb, out, "separable")
    for _ in range(3):
        run()
    torch.cuda.synchronize()
    check(img, kb, out.cpu().numpy())


def test_l2_flush_and_tuner_without_mutation():
    """sepconv_l2_flush is measurement hygiene: it launches no SeparableConvolution kernel (the
    launch counter does not move) and leaves results untouched; a tune with the mutation search
    off returns the model's schedule (no override), a tuned pick with it on is still one of the
    candidates, and both match the oracle."""
    h, w, K = 900, 1300, 7
    img = synth.uniform_image(h, w, seed=12)
    k = synth.binomial_kernel(K)
    before = sc.launch_count()
    for _ in range(3):
        sc.l2_flush()
    torch.cuda.synchronize()
    assert sc.launch_count() == before
    p = sc.Plan(h, w, K)
    plain = p.tune(reps=3, force=True, mutations=-1)
    assert plain.sched_parts == 0 and plain.sched_grid == 0 and plain.source == sc.SRC_TUNED
    check(img, k, run_gpu(img, k, variant="auto", plan=p)[0])
    mutated = p.tune(reps=3, force=True, mutations=6, seed=3)
    assert mutated.base_name in {c.name for c in p.candidates()}
    check(img, k, run_gpu(img, k, variant="auto", plan=p)[0])


def test_band_timeline_orders_the_phases():
    """sepconv_band_trace / sepconv_band_timeline (the overlap evidence of SURVEY 8(e)): on a
    middle band in external-halo mode the interior kernel, the (empty) exchange and the tail
    kernel are timed on the device; the tail starts after the interior ends and after the
    exchange event, every interval is non-negative, and tracing changes no output bit."""
    H, W, K, G, g = 3000, 4096, 9, 3, 1
    img = torch.from_numpy(synth.uniform_image(H, W, seed=43)).cuda()
    k = synth.binomial_kernel(K)
    r0, rows, owned, alloc = sc.band(H, K, G, g)
    band = img[r0:r0 + alloc].clone()
    p = sc.Plan(alloc, W, K)
    p.comm_init(None, G, g)
    with pytest.raises(sc.SepconvError):
        p.band_timeline()                                 # tracing off
    out0 = torch.empty((rows, W - K + 1), device="cuda")
    p.run_band(band, k, out0)
    p.band_trace(True)
    out1 = torch.empty_like(out0)
    p.run_band(band, k, out1)
    tl = p.band_timeline()
    (i0, i1), (x0, x1), (t0, t1) = tl["interior"], tl["exchange"], tl["tail"]
    assert 0 <= i0 <= i1 and 0 <= x0 <= x1 and 0 <= t0 <= t1
    assert t0 >= i1 and t0 >= x1 and i1 - i0 > 0 and t1 - t0 > 0
    assert torch.equal(out0, out1)


def test_run_band_nccl_single_rank_and_shared_comm():
    """The NCCL path end to end on one GPU: the library dlopens the process's libnccl,
    creates a unique id and a 1-rank communicator (no peers, so no send/recv is posted),
    shares it between two plans, and run_band equals a plain run."""
    H, W, K = 300, 700, 7
    img = torch.from_numpy(synth.uniform_image(H, W, seed=41)).cuda()
    k = synth.binomial_kernel(K)
    uid = sc.nccl_unique_id()
    assert len(uid) == sc.NCCL_ID_BYTES
    p1, p2 = sc.Plan(H, W, K), sc.Plan(H, W, K)
    p1.comm_init(uid, 1, 0)
    p2.comm_init(uid, 1, 0)                               # same id: shared communicator
    want = torch.empty((H - K + 1, W - K + 1), device="cuda")
    p1.run(img, k, want, "separable")
    for p in (p1, p2):
        got = torch.empty_like(want)
        band = img.clone()
        p.run_band(band, k, got, "separable")
        torch.cuda.synchronize()
        assert torch.equal(got, want)
    p1.close()
    p2.close()


def test_size_selector_resolves_untuned_plans(tmp_path, monkeypatch):
    """NEXT-2: sepconv_tune_selector builds SELECT's cutoff table for K over the 12 default
    square levels and stores it in the tuning cache; a plan of an
    untuned shape (3000^2, between the 2048 and 3072 levels) then resolves AUTO through it
    (source SELECTOR, the same choice sepconv_select gives for 3000^2 pixels) and matches the
    oracle on the whole output.  A shape with its own tuned entry still takes that entry."""
    cache = str(tmp_path / "tune.jsonl")
    K = 9
    sel = sc.tune_selector(K, reps=5, cache_path=cache)
    assert 1 <= len(sel.algos) <= 12 and len(sel.cutoffs) == len(sel.algos) - 1
    assert all(a < b for a, b in zip(sel.cutoffs, sel.cutoffs[1:]))
    assert all(64 * 64 < c < 16384 * 16384 for c in sel.cutoffs)
    monkeypatch.setenv("SEPCONV_TUNE_CACHE", cache)
    p = sc.Plan(3000, 3000, K)
    got = p.get_choice("auto")
    want = sel.select(3000 * 3000)
    assert got.source == sc.SRC_SELECTOR and got.base_name == want.base_name, (got, want, sel)
    img = synth.uniform_image(3000, 3000, seed=5)
    k = synth.binomial_kernel(K)
    check(img, k, run_gpu(img, k, variant="auto", plan=p)[0])
    # an exact tuned entry wins over the selector
    q = sc.Plan(512, 640, K)
    q.tune(reps=3, cache_path=cache, force=True)
    assert sc.Plan(512, 640, K).get_choice("auto").source == sc.SRC_TUNED


def test_mutated_schedules_are_bitwise_equal_and_tuned_one_is_kept(tmp_path):
    """Schedule overrides (the size-like tunables the mutation search scales) change
    which CTA computes which rows, never a pixel's arithmetic (R6): every
    (parts, grid) gives the model schedule's bits.  The tuner's mutated AUTO pick round-trips
    through the cache and passes parity."""
    h, w, K = 1500, 2300, 13
    img = synth.uniform_image(h, w, seed=8)
    k = synth.random_kernel(K, seed=3, signed=True)
    p = sc.Plan(h, w, K)
    dev = torch.from_numpy(img).cuda()
    base = sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 2)
    ref = torch.empty((h - K + 1, w - K + 1), device="cuda")
    p.run_choice(dev, k, ref, base)
    for parts, grid in ((1, 1), (1, 3), (7, 20), (40, 148), (3000, 148), (13, 0), (200, 37)):
        out = torch.full_like(ref, float("nan"))
        p.run_choice(dev, k, out, sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 2, sched_parts=parts,
                                            sched_grid=grid))
        torch.cuda.synchronize()
        assert torch.equal(out, ref), (parts, grid)
    for c in (sc.Choice(sc.SEPCONV_2D, sc.MAP_TMA, 0, sched_parts=5, sched_grid=60),):
        out = torch.full_like(ref, float("nan"))
        p.run_choice(dev, k, out, c)
        torch.cuda.synchronize()
        check(img, k, out.cpu().numpy())
    cache = str(tmp_path / "t.jsonl")
    best = p.tune(reps=5, cache_path=cache, force=True, mutations=16, seed=7)
    assert sc.Plan(h, w, K).tune(reps=5, cache_path=cache) == best
    check(img, k, run_gpu(img, k, variant="auto", plan=p)[0])


@pytest.mark.parametrize("n,h,w,K,cfg,parts,grid", [
    (1, 2048, 2048, 17, 2, 74, 0),     # 2 strips x 74 parts = 148 segments, one per CTA
    (1, 2048, 2048, 17, 4, 70, 0),     # 140 segments on 148 slots
    (1, 2048, 2048, 17, 5, 74, 0),     # 4-warp CTAs, 2 per SM: 4 strips x 74 = 296 segments
    (1, 2048, 2048, 17, 2, 300, 148),  # 600 segments, ~4 per CTA
    (1, 2048, 2048, 17, 2, 5, 7),      # few long segments: thieves split them repeatedly
    (1, 2048, 2048, 17, 0, 74, 0),     # lockstep stages: stealing compiled out, override applies
    (1, 2048, 2048, 17, 3, 148, 0),    # 16 warps: likewise
    (3, 601, 700, 9, 2, 49, 0),        # a batch, ragged 700-column strip
    (1, 1000, 3000, 5, 4, 9, 20),      # 3 strips, the last one ragged; K=5 (stage = 10 rows)
    (1, 1000, 3000, 3, 5, 40, 0),      # K=3 (stage = 6 rows)
])
def test_work_stealing_bitwise(n, h, w, K, cfg, parts, grid):
    """Work stealing between warps (sched_steal, R27) moves the unclaimed stages of a
    warp's rows to whichever warp runs out of work first; it changes no pixel's arithmetic, so
    every threshold gives the model schedule's bits, on repeated launches (a fresh claim epoch
    each, through the replay fast path) that reuse the same claim words."""
    img = synth.uniform_image(n * h, w, seed=31).reshape(n, h, w)
    k = synth.random_kernel(K, seed=5, signed=True)
    p = sc.Plan(h, w, K, n=n)
    dev = torch.from_numpy(img).cuda()
    ref = torch.empty((n, h - K + 1, w - K + 1), device="cuda")
    p.run_choice(dev, k, ref, sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg))
    torch.cuda.synchronize()
    for i in range(n):
        check(img[i], k, ref[i].cpu().numpy())
    for steal in (1, 2, 4, 16, 99, 4):
        c = sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, sched_parts=parts, sched_grid=grid,
                      sched_steal=steal)
        assert c.name.endswith("st%d" % steal)
        for _ in range(3):
            out = torch.full_like(ref, float("nan"))
            p.run_choice(dev, k, out, c)
            torch.cuda.synchronize()
            assert torch.equal(out, ref), (steal, c.name)


# ---- work schedules: the window schedule (every SM busy) equals the others bit for bit -----
@pytest.mark.parametrize("choice", [CANDS[i] for i in (0, 2, 3, 4, 5, 7, 8, 10)],
                         ids=[IDS[i] for i in (0, 2, 3, 4, 5, 7, 8, 10)])
def test_window_schedule_bitwise_and_parity(choice, monkeypatch):
    """SEPCONV_SCHED=win forces the window schedule (q full-width windows + CTAs sharing the
    short last window) wherever it is eligible; the schedule changes no pixel's arithmetic
    (R6), so the output equals the strided/contiguous schedules' bitwise, and it
    matches the oracle.  5 strips of 1024 columns on 148 SMs: q = 29, e = 3, m = 2."""
    h, w = 2600, 5000
    img = synth.uniform_image(h, w, seed=77)
    dev = torch.from_numpy(img).cuda()
    for K in (3, 10, 17):
        k = synth.random_kernel(K, seed=K, signed=True)
        p = sc.Plan(h, w, K)
        outs = {}
        for mode in ("nowin", "win"):
            monkeypatch.setenv("SEPCONV_SCHED", mode)
            out = torch.full((h - K + 1, w - K + 1), float("nan"), device="cuda")
            p.run_choice(dev, k, out, choice)
            torch.cuda.synchronize()
            outs[mode] = out
        monkeypatch.delenv("SEPCONV_SCHED")
        assert not torch.isnan(outs["win"]).any().item(), f"K={K}: a cell was not written"
        assert torch.equal(outs["win"], outs["nowin"]), f"K={K}"
        rows = sorted({0, 1, 87, 88, 1000, h - K - 40, h - K - 1, h - K})
        got = outs["win"][rows].cpu().numpy()
        for i, r in enumerate(rows):
            o, s = oracle.convolve2d(np.ascontiguousarray(img[r:r + K]), k, with_absum=True)
            assert rel_error(got[i:i + 1], o, s) <= TOL, (K, r)
        p.close()
