"""GPU parity: the CUDA path (through the C-ABI) vs the CPU oracle, element by element.

Integer work, so the bar is bit-exact: matches and checksum equal, materialized pairs equal
after a lexicographic sort (reading S9), partitions equal as multisets. Inputs are the seeded
generator's (workloads/) or small adversarial arrays; expected values come only from oracle/
or from the generator's closed forms, never from the CUDA path.
"""
import ctypes
import os

import numpy as np
import pytest
import torch

import oracle
import workloads as W

pytestmark = pytest.mark.gpu

M64 = (1 << 64) - 1
GOLDEN = 0x9E3779B97F4A7C15


@pytest.fixture(scope="module")
def hj():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as m

    return m


def dev(a: np.ndarray):
    t = torch.from_numpy(np.ascontiguousarray(a).view(np.int32 if a.dtype.itemsize == 4 else np.int64))
    return t.cuda()


def np_sig(p, q):
    with np.errstate(over="ignore"):
        return W.np_fmix64(p.astype(np.uint64) ^ (q.astype(np.uint64) * np.uint64(GOLDEN)))


def gpu_join(hj, Rk, Rp, Sk, Sp, bits=-1, mat=False, ctx=None):
    c = ctx or hj.context(0, Rk.dtype.itemsize, Rp.dtype.itemsize)
    res = c.join(dev(Rk), dev(Rp), dev(Sk), dev(Sp), radix_bits=bits,
                 out_mode=hj.OUT_MATERIALIZE if mat else hj.OUT_COUNT_CHECKSUM)
    torch.cuda.synchronize()
    return res


def to_np(t, width):
    return t.cpu().numpy().view(np.uint32 if width == 4 else np.uint64)


def check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=-1, mat=True, ctx=None):
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    res = gpu_join(hj, Rk, Rp, Sk, Sp, bits, mat=False, ctx=ctx)
    assert (res.matches, res.checksum) == (m, c), f"count mode bits={bits}"
    if mat:
        res = gpu_join(hj, Rk, Rp, Sk, Sp, bits, mat=True, ctx=ctx)
        assert res.matches == m, f"materialize mode bits={bits}"
        assert res.checksum == c, f"materialize-mode checksum bits={bits}"  # HJ_OPT_MAT_CHECKSUM = 1
        if m:
            w = Rp.dtype.itemsize
            got = oracle.pairs_sorted(to_np(res.r_pay, w), to_np(res.s_pay, w))
            assert np.array_equal(got, oracle.pairs_sorted(r, s))
            # the aggregate recomputed on the host from the returned pairs equals the oracle's
            assert int(np_sig(got[:, 0], got[:, 1]).sum(dtype=np.uint64)) == c
    return res


def adversarial(rng):
    u32 = np.uint32
    return {
        "all_equal": (np.full(300, 5, u32), np.full(200, 5, u32)),
        "disjoint": (np.arange(0, 5000, 2, dtype=u32), np.arange(1, 5001, 2, dtype=u32)),
        "dups_both": (rng.integers(0, 40, 700).astype(u32), rng.integers(0, 40, 900).astype(u32)),
        "extremes": (np.array([0, 0xFFFFFFFF, 1, 0xFFFFFFFE] * 3, u32), np.array([0xFFFFFFFF, 0, 0, 7], u32)),
        "high_bits_only": ((np.arange(3000, dtype=u32) << u32(20)) | u32(3),
                           (np.arange(0, 6000, dtype=u32) << u32(19)) | u32(3)),
        "one_row": (np.array([42], u32), np.array([42, 42, 1], u32)),
        "random_ragged": (rng.integers(0, 300000, 40961).astype(u32), rng.integers(0, 300000, 30011).astype(u32)),
        "sparse_uniform": (rng.integers(0, 1 << 32, 100003, dtype=np.uint64).astype(u32),
                           rng.integers(0, 1 << 32, 77777, dtype=np.uint64).astype(u32)),
    }


CASES = list(adversarial(np.random.default_rng(0)).keys())


@pytest.mark.parametrize("name", CASES)
@pytest.mark.parametrize("bits", [-1, 0, 1, 2, 5, 8, 13])
def test_adversarial_vs_oracle(hj, name, bits):
    rng = np.random.default_rng(99)
    Rk, Sk = adversarial(rng)[name]
    Rp = rng.integers(0, 1 << 32, len(Rk), dtype=np.uint64).astype(np.uint32)
    Sp = rng.integers(0, 1 << 32, len(Sk), dtype=np.uint64).astype(np.uint32)
    check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=bits, mat=True)


def test_empty_inputs(hj):
    z = np.zeros(0, np.uint32)
    a = np.arange(10, dtype=np.uint32)
    for Rk, Sk in [(z, a), (a, z), (z, z)]:
        res = gpu_join(hj, Rk, Rk.copy(), Sk, Sk.copy(), mat=True)
        assert (res.matches, res.checksum) == (0, 0)


@pytest.mark.parametrize("cap_r,chunk_s", [(7, 0), (100, 33), (0, 1), (513, 4097), (4096, 5)])
def test_knob_invariance_block_nested_loops(hj, cap_r, chunk_s):
    """Tiny C_R forces hash-based block nested loops; tiny C_S forces S splitting
    (P:306-308). Results must not change."""
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_CAP_R, cap_r)
    ctx.set_option(hj.OPT_CHUNK_S, chunk_s)
    rng = np.random.default_rng(5)
    Rk = rng.integers(0, 3000, 20000).astype(np.uint32)
    Sk = rng.integers(0, 3000, 15000).astype(np.uint32)
    Rp = np.arange(len(Rk), dtype=np.uint32)
    Sp = np.arange(len(Sk), dtype=np.uint32)
    for bits in (0, 4, 9):
        check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=bits, mat=True, ctx=ctx)
    ctx.close()


JOIN_SHAPES = 9  # number of k_join shapes in hj_api.cu (HJ_OPT_JOIN_VARIANT 1..9)


@pytest.mark.parametrize("variant", range(1, JOIN_SHAPES + 1))
def test_join_shape_invariance(hj, variant):
    """Every selectable join-kernel shape (block size, tuples per thread, blocks/SM, R buffers,
    hash-slot count, 16-bit heads) gives the oracle's result, on skewed and duplicate-heavy keys,
    4- and 8-byte tuples."""
    rng = np.random.default_rng(40 + variant)
    for kb in (4, 8):
        ctx = hj.Context(0, kb, kb)
        ctx.set_option(hj.OPT_JOIN_VARIANT, variant)
        dt = np.uint32 if kb == 4 else np.uint64
        w = W.Workload("v", 30011, 50021, "zipf", keys="sparse" if kb == 4 else "k8", z=1.2, seed=400 + variant)
        Rk, Rp, Sk, Sp = W.np_generate(w)
        for bits in (-1, 2, 7):
            check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=bits, mat=True, ctx=ctx)
        Rk = rng.integers(0, 700, 9000).astype(dt)
        Sk = rng.integers(0, 700, 7000).astype(dt)
        check_against_oracle(hj, Rk, np.arange(len(Rk), dtype=dt), Sk, np.arange(len(Sk), dtype=dt), bits=3,
                             mat=True, ctx=ctx)
        ctx.close()
    with pytest.raises(Exception):
        hj.Context(0, 4, 4).set_option(hj.OPT_JOIN_VARIANT, JOIN_SHAPES + 1)


def _bc_ctx(hj, kb=4, **opts):
    ctx = hj.Context(0, kb, kb)
    ctx.set_option(hj.OPT_PARTITIONER, 1)
    for k, v in opts.items():
        ctx.set_option(getattr(hj, k), v)
    return ctx


@pytest.mark.parametrize("name", CASES)
@pytest.mark.parametrize("bits", [-1, 0, 1, 5, 13])
def test_bucket_chains_adversarial(hj, name, bits):
    """NEXT-1 (HJ_OPT_PARTITIONER = 1, the paper's histogram-free bucket chains)
    gives the oracle's result on the adversarial inputs."""
    rng = np.random.default_rng(98)
    Rk, Sk = adversarial(rng)[name]
    Rp = rng.integers(0, 1 << 32, len(Rk), dtype=np.uint64).astype(np.uint32)
    Sp = rng.integers(0, 1 << 32, len(Sk), dtype=np.uint64).astype(np.uint32)
    ctx = _bc_ctx(hj)
    check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=bits, mat=True, ctx=ctx)
    ctx.close()


@pytest.mark.parametrize("cfg", [
    dict(nR=1 << 18, nS=1 << 20, dist="fk", keys="sparse", bits=2),   # pass-1 buckets close many times
    dict(nR=1 << 16, nS=1 << 20, dist="zipf", z=1.5, keys="sparse", bits=8),  # a hot co-partition: long pass-2 chains
    dict(nR=100_003, nS=300_007, dist="zipf_build", z=1.0, keys="dense", bits=6),
    dict(nR=1 << 15, nS=1 << 15, dist="replicas", rep=4, keys="dense", bits=4),
    dict(nR=70_001, nS=90_001, dist="fk", keys="k8", bits=7),
    dict(nR=1 << 17, nS=1 << 17, dist="1to1", keys="dense", bits=-1),
])
def test_bucket_chains_generated(hj, cfg):
    cfg = dict(cfg)
    bits = cfg.pop("bits")
    w = W.Workload("bc", seed=500 + cfg["nR"] % 97, **cfg)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    ctx = _bc_ctx(hj, w.key_bytes)
    check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=bits, mat=True, ctx=ctx)
    ctx.close()


@pytest.mark.parametrize("kb", [4, 8])
@pytest.mark.parametrize("bits", [6, 10])
def test_bucket_chains_growing_regions(hj, kb, bits):
    """Pass 2's growing regions (hj_bucket.cuh: 1, 1, 2, 4, 8, 16, 16, .. consecutive buckets per
    overflow): one key carries 3/4 of S, so its co-partition closes hundreds of buckets and its
    regions reach 16 buckets; a few other keys close a couple each. The pool bound must hold
    (an overflow raises) and the result equals the oracle's, with and without materialization."""
    dt = np.uint32 if kb == 4 else np.uint64
    rng = np.random.default_rng(77)
    nS = 1 << 21
    Sk = rng.integers(0, 1 << 20, nS).astype(dt)
    Sk[rng.random(nS) < 0.75] = 123457
    Sk[rng.random(nS) < 0.02] = 99991
    Rk = np.concatenate([rng.integers(0, 1 << 20, 1 << 16).astype(dt), np.array([123457, 99991, 99991], dt)])
    Rp = np.arange(len(Rk), dtype=dt)
    Sp = rng.integers(0, 1 << 31, nS).astype(dt)
    ctx = _bc_ctx(hj, kb)
    check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=bits, mat=True, ctx=ctx)
    ctx.close()


@pytest.mark.parametrize("cap_r,chunk_s", [(7, 0), (100, 33), (4096, 5)])
def test_bucket_chains_slices(hj, cap_r, chunk_s):
    """Tiny C_R / C_S cut the final buckets into many join slices (block nested loops)."""
    rng = np.random.default_rng(6)
    Rk = rng.integers(0, 3000, 20000).astype(np.uint32)
    Sk = rng.integers(0, 3000, 15000).astype(np.uint32)
    ctx = _bc_ctx(hj, OPT_CAP_R=cap_r, OPT_CHUNK_S=chunk_s, OPT_OUT_CAPACITY=1000)
    for bits in (0, 4, 9):
        check_against_oracle(hj, Rk, np.arange(len(Rk), dtype=np.uint32), Sk, np.arange(len(Sk), dtype=np.uint32),
                             bits=bits, mat=True, ctx=ctx)
    ctx.close()


def test_bucket_chains_equal_histogram_path_and_repeat(hj):
    """Same ctx, alternating partitioners and repeated calls: identical results (no state leaks
    between calls through the pools or the zeroed metadata)."""
    w = W.Workload("bc2", 1 << 19, 1 << 21, "zipf", z=1.0, keys="sparse", seed=510)
    cols = [dev(a) for a in W.np_generate(w)]
    ctx = hj.Context(0, 4, 4)
    ref = oracle.hash_join(*W.np_generate(w))
    for part in (1, 0, 1, 1):
        ctx.set_option(hj.OPT_PARTITIONER, part)
        r = ctx.join(*cols)
        torch.cuda.synchronize()
        assert (r.matches, r.checksum) == ref, part
    ctx.close()


def test_materialize_overflow_regrows(hj):
    """More matches than the initial capacity: grow and re-run the join phase (reading S11)."""
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_OUT_CAPACITY, 1000)
    Rk = np.repeat(np.arange(50, dtype=np.uint32), 40)
    Sk = np.repeat(np.arange(60, dtype=np.uint32), 30)
    Rp = np.arange(len(Rk), dtype=np.uint32)
    Sp = np.arange(len(Sk), dtype=np.uint32)
    res = check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=3, mat=True, ctx=ctx)
    assert res.matches == 50 * 40 * 30
    ctx.close()


@pytest.mark.parametrize("dist,keys,z", [("fk", "dense", 0), ("1to1", "sparse", 0), ("zipf", "dense", 1.5),
                                         ("zipf", "sparse", 1.0), ("fk", "k8", 0), ("1to1", "k8", 0)])
@pytest.mark.parametrize("nR,nS", [(1 << 16, 1 << 18), (40000, 70001)])
def test_generated_vs_oracle(hj, dist, keys, z, nR, nS):
    if dist == "1to1":
        nS = nR
    w = W.Workload("t", nR, nS, dist, keys=keys, z=z, seed=120)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=-1, mat=True)


def test_8byte_adversarial(hj):
    rng = np.random.default_rng(8)
    Rk = rng.integers(0, 500, 30000, dtype=np.uint64) * np.uint64(0x100000001) + np.uint64(1 << 62)
    Sk = rng.integers(0, 600, 20000, dtype=np.uint64) * np.uint64(0x100000001) + np.uint64(1 << 62)
    Rp = rng.integers(0, 1 << 63, len(Rk), dtype=np.uint64)
    Sp = rng.integers(0, 1 << 63, len(Sk), dtype=np.uint64)
    for bits in (0, 3, 10):
        check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=bits, mat=True)


@pytest.mark.parametrize("bits", [0, 1, 6, 11, 15])
@pytest.mark.parametrize("width", [4, 8])
def test_partition_vs_oracle(hj, bits, width):
    """Steps a1-a4: every co-partition holds exactly the oracle's multiset of tuples."""
    rng = np.random.default_rng(bits + width)
    dt = np.uint32 if width == 4 else np.uint64
    n = 300_001
    keys = rng.integers(0, 1 << (8 * width - 1), n, dtype=np.uint64).astype(dt)
    pays = np.arange(n, dtype=dt)
    ok, op, offs = oracle.radix_partition(keys, pays, 0, bits)
    ctx = hj.context(0, width, width)
    t, start, count = ctx.partition(dev(keys), dev(pays), bits)
    torch.cuda.synchronize()
    assert np.array_equal(count, np.diff(offs.astype(np.int64)).astype(np.uint64))
    tt = t.cpu().numpy()
    if width == 4:
        gk = (tt.view(np.uint64) & np.uint64(0xFFFFFFFF)).astype(np.uint32)
        gp = (tt.view(np.uint64) >> np.uint64(32)).astype(np.uint32)
    else:
        gk = tt[:, 0].view(np.uint64)
        gp = tt[:, 1].view(np.uint64)
    # the partitions tile [0, n) and each equals the oracle's multiset
    order = np.argsort(start, kind="stable")
    assert start[order[0]] == 0
    for p in range(1 << bits):
        a, c = int(start[p]), int(count[p])
        o0 = int(offs[p])
        g = np.sort(gp[a:a + c])
        e = np.sort(op[o0:o0 + c])
        assert np.array_equal(g, e), f"partition {p}"
        assert np.all((gk[a:a + c] & dt((1 << bits) - 1)) == p)
    # key <-> payload pairing survives both passes (payloads are row ids)
    assert np.array_equal(gk, keys[gp.astype(np.int64)])
    assert int(start.max() + count[np.argmax(start)]) <= n


@pytest.mark.parametrize("bits", [8, 11, 15])
@pytest.mark.parametrize("width", [4, 8])
def test_partition_skewed_vs_oracle(hj, bits, width):
    """Steps a1-a4 on skewed keys: the planner's hot-digit hints (one pass-1 digit with > 1/4 of
    a relation, one d2 digit with > 1/4 of a pass-1 partition) switch the passes to ballot ranking
    for those digits; the partitions must still equal the oracle's multisets."""
    rng = np.random.default_rng(300 + bits + width)
    dt = np.uint32 if width == 4 else np.uint64
    n = 400_003
    keys = rng.integers(0, 1 << (8 * width - 1), n, dtype=np.uint64).astype(dt)
    u = rng.random(n)
    keys[u < 0.40] = dt(0x5A5A5A5A)          # > 1/4 of the relation: a pass-1 hint
    keys[(u >= 0.40) & (u < 0.55)] = dt(77)  # 15 %: its pass-1 partition is mostly one d2 digit
    pays = np.arange(n, dtype=dt)
    ok, op, offs = oracle.radix_partition(keys, pays, 0, bits)
    ctx = hj.context(0, width, width)
    t, start, count = ctx.partition(dev(keys), dev(pays), bits)
    torch.cuda.synchronize()
    assert np.array_equal(count, np.diff(offs.astype(np.int64)).astype(np.uint64))
    tt = t.cpu().numpy()
    if width == 4:
        gk = (tt.view(np.uint64) & np.uint64(0xFFFFFFFF)).astype(np.uint32)
        gp = (tt.view(np.uint64) >> np.uint64(32)).astype(np.uint32)
    else:
        gk = tt[:, 0].view(np.uint64)
        gp = tt[:, 1].view(np.uint64)
    for p in range(1 << bits):
        a, c = int(start[p]), int(count[p])
        o0 = int(offs[p])
        assert np.array_equal(np.sort(gp[a:a + c]), np.sort(op[o0:o0 + c])), f"partition {p}"
    assert np.array_equal(gk, keys[gp.astype(np.int64)])


def test_join_host_matches_device(hj):
    w = W.Workload("t", 1 << 15, 1 << 16, "fk", seed=121)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    res = hj.join_host(Rk, Rp, Sk, Sp, out_mode=hj.OUT_MATERIALIZE)
    assert res.matches == m
    assert hj.join_host(Rk, Rp, Sk, Sp).checksum == c
    assert np.array_equal(oracle.pairs_sorted(res.r_pay, res.s_pay), oracle.pairs_sorted(r, s))


def test_c1_full_size_vs_oracle(hj):
    """BASELINE config[0]: FK 1M ⋈ 1M, count + checksum, element by element vs the oracle."""
    w = W.CONFIGS["c1"]
    Rk, Rp, Sk, Sp = W.np_generate(w)
    check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=w.radix_bits, mat=True)


def test_device_generator_matches_host(hj):
    w = W.Workload("t", 1 << 18, 1 << 19, "zipf", z=1.5, seed=122)
    a = W.np_generate(w)
    b = W.torch_generate(w, device="cuda")
    for x, y in zip(a, b):
        assert np.array_equal(x, to_np(y, x.dtype.itemsize))


@pytest.mark.slow
@pytest.mark.parametrize("cfg", ["c2", "c3", "c4_z0.5", "c4_z1.0", "c4_z1.5", "c5_gpu"])
def test_full_size_closed_form(hj, cfg):
    """Full BASELINE sizes in the bench's launch configuration: matches == |S| and the checksum
    equals sum_j sig(rho(j), j) computed on the host from the generator (closed form); for c3's
    materialized output, the pairs sorted by s_pay are exactly (rho(j), j)."""
    w = W.CONFIGS[cfg]
    Rk, Rp, Sk, Sp = W.torch_generate(w, device="cuda")
    cdf = W.zipf_cdf(w.nR, w.z) if w.dist == "zipf" else None
    # the device-generated inputs equal the host generator on a sample of rows
    rows = np.random.default_rng(0).integers(0, w.nS, 1 << 16).astype(np.uint64)
    rho_s = W.np_rho_for(w, rows, cdf)
    Rk_h = W.np_generate(w, s_rows=slice(0, 0))[0]  # R keys only
    kb = w.key_bytes
    assert np.array_equal(to_np(Sk[torch.from_numpy(rows.astype(np.int64)).cuda()], kb), Rk_h[rho_s.astype(np.int64)]), \
        "device generator differs from the host generator"
    del Rk_h
    ctx = hj.context(0, kb, kb)
    res = ctx.join(Rk, Rp, Sk, Sp, radix_bits=w.radix_bits, out_mode=w.out_mode)
    torch.cuda.synchronize()
    del Rk, Rp, Sk, Sp
    j = np.arange(w.nS, dtype=np.uint64)
    rho = W.np_rho_for(w, j, cdf)
    assert res.matches == w.nS, f"matches {res.matches} != |S| {w.nS} (items {res.n_items})"
    exp = int(np_sig(rho, j).sum(dtype=np.uint64))  # both modes (materialize: HJ_OPT_MAT_CHECKSUM)
    assert res.checksum == exp, f"checksum {res.checksum:#x} != closed form {exp:#x} (items {res.n_items})"
    if w.out_mode == 1:
        s_pay = res.s_pay
        order = torch.argsort(s_pay)
        r_sorted = to_np(res.r_pay[order], kb).astype(np.uint64)
        s_sorted = to_np(s_pay[order], kb).astype(np.uint64)
        assert np.array_equal(s_sorted, j), "materialized s_pay is not a permutation of S's rows"
        bad = np.nonzero(r_sorted != rho)[0]
        assert len(bad) == 0, f"{len(bad)} materialized pairs differ, first at s_pay {bad[:5]}"


@pytest.mark.slow
@pytest.mark.parametrize("slice_id", [0, 11])
def test_c5_shape_sliced_oracle(hj, slice_id):
    """c5's shape (1:1, 8-byte fmix64 keys, row-id payloads, B = 16 local bits) at 2^26 x 2^26
    rows: the oracle's sliced mode (slice = top 4 bits of fmix64(key); the join decomposes over any
    key partition) on one slice equals the GPU join of that slice's rows, and the GPU
    join of all rows equals the closed form."""
    w = W.Workload("c5s", 1 << 26, 1 << 26, "1to1", keys="k8", seed=107, out_mode=0, radix_bits=16)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    bits = 4
    m, c = oracle.hash_join(Rk, Rp, Sk, Sp, slice_bits=bits, slice_id=slice_id)
    inR = (W.np_fmix64(Rk) >> np.uint64(64 - bits)) == np.uint64(slice_id)
    inS = (W.np_fmix64(Sk) >> np.uint64(64 - bits)) == np.uint64(slice_id)
    assert m == int(inS.sum()) and m > (1 << 21)
    res = gpu_join(hj, Rk[inR], Rp[inR], Sk[inS], Sp[inS], bits=12)
    assert (res.matches, res.checksum) == (m, c)
    full = gpu_join(hj, Rk, Rp, Sk, Sp, bits=w.radix_bits)
    assert (full.matches, full.checksum) == (w.nS, _closed_form_checksum(w))


@pytest.mark.parametrize("width", [4, 8])
def test_partition_16bit_counters_wrap(hj, width):
    """2^16 co-partitions use packed 16-bit shared-memory counters; > 65535 equal keys in one
    block exercise the wrap/carry correction."""
    rng = np.random.default_rng(16)
    dt = np.uint32 if width == 4 else np.uint64
    n = 400_000
    keys = rng.integers(0, 1 << (8 * width - 1), n, dtype=np.uint64).astype(dt)
    keys[: 3 * n // 4] = dt(0x12345)  # 300K copies of one key
    rng.shuffle(keys)
    pays = np.arange(n, dtype=dt)
    _, _, offs = oracle.radix_partition(keys, pays, 0, 16)
    t, start, count = hj.context(0, width, width).partition(dev(keys), dev(pays), 16)
    torch.cuda.synchronize()
    assert np.array_equal(count, np.diff(offs.astype(np.int64)).astype(np.uint64))


@pytest.mark.parametrize("width", [4, 8])
def test_partition_16bit_counters_two_hot_bins_one_word(hj, width):
    """2^16 bins are packed two per 32-bit word: two hot keys whose bins share a word (bins 2k and
    2k + 1), each far past 65535 occurrences in one histogram block, interleaved so both halves
    wrap repeatedly while the other is being incremented (a carry between the halves
    must never be visible to the partner bin)."""
    rng = np.random.default_rng(18)
    dt = np.uint32 if width == 4 else np.uint64
    n = 1_200_000
    keys = rng.integers(0, 1 << (8 * width - 1), n, dtype=np.uint64).astype(dt)
    hot = rng.random(n)
    keys[hot < 0.45] = dt(0x52344)   # bin 0x2344 (even)
    keys[(hot >= 0.45) & (hot < 0.9)] = dt(0x72345)  # bin 0x2345 (odd): same packed word
    pays = np.arange(n, dtype=dt)
    _, _, offs = oracle.radix_partition(keys, pays, 0, 16)
    t, start, count = hj.context(0, width, width).partition(dev(keys), dev(pays), 16)
    torch.cuda.synchronize()
    assert np.array_equal(count, np.diff(offs.astype(np.int64)).astype(np.uint64))


def test_join_16bit_counters(hj):
    rng = np.random.default_rng(17)
    Rk = rng.integers(0, 1 << 20, 150_000).astype(np.uint32)
    Sk = np.concatenate([rng.integers(0, 1 << 20, 100_000), np.full(90_000, Rk[7])]).astype(np.uint32)
    Rp = np.arange(len(Rk), dtype=np.uint32)
    Sp = np.arange(len(Sk), dtype=np.uint32)
    check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=16, mat=True)


@pytest.mark.parametrize("chunk", [1000, 4097, 65536])
@pytest.mark.parametrize("dist_", ["fk", "zipf"])
def test_join_host_streaming_vs_oracle(hj, chunk, dist_):
    """NEXT-3 streaming probe: S copied and joined in chunks against the resident R;
    the union of the chunk joins is the join."""
    w = W.Workload("t", 30_000, 200_003, dist_, keys="sparse", z=1.0, seed=150)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_STREAM_CHUNK, chunk)
    res = ctx.join_host(Rk, Rp, Sk, Sp)
    assert (res.matches, res.checksum) == (m, c)
    res = ctx.join_host(Rk, Rp, Sk, Sp, out_mode=hj.OUT_MATERIALIZE)
    assert res.matches == m
    assert np.array_equal(oracle.pairs_sorted(res.r_pay, res.s_pay), oracle.pairs_sorted(r, s))
    ctx.close()


def test_join_host_streaming_duplicates_and_overflow(hj):
    """Duplicate keys on both sides; the result outgrows the initial output capacity, so the
    streamed call falls back to the copy-everything path and regrows (reading S11)."""
    rng = np.random.default_rng(151)
    Rk = rng.integers(0, 300, 5000).astype(np.uint32)
    Sk = rng.integers(0, 300, 20000).astype(np.uint32)
    Rp = np.arange(len(Rk), dtype=np.uint32)
    Sp = np.arange(len(Sk), dtype=np.uint32)
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_STREAM_CHUNK, 3000)
    ctx.set_option(hj.OPT_OUT_CAPACITY, 50_000)
    res = ctx.join_host(Rk, Rp, Sk, Sp, out_mode=hj.OUT_MATERIALIZE)
    assert res.matches == m > 50_000
    assert np.array_equal(oracle.pairs_sorted(res.r_pay, res.s_pay), oracle.pairs_sorted(r, s))
    assert ctx.join_host(Rk, Rp, Sk, Sp).checksum == c
    ctx.close()


def test_join_host_streaming_8byte(hj):
    w = W.Workload("t", 1 << 14, 1 << 17, "fk", keys="k8", seed=152)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    m, c = oracle.hash_join(Rk, Rp, Sk, Sp)
    ctx = hj.Context(0, 8, 8)
    ctx.set_option(hj.OPT_STREAM_CHUNK, 10_000)
    assert (lambda r: (r.matches, r.checksum))(ctx.join_host(Rk, Rp, Sk, Sp)) == (m, c)
    ctx.close()


@pytest.mark.parametrize("algo", [1, 2])
@pytest.mark.parametrize("name", ["all_equal", "dups_both", "extremes", "random_ragged", "sparse_uniform", "one_row"])
def test_comparator_algorithms_vs_oracle(hj, algo, name):
    """NEXT-4: the ballot nested-loop co-partition join (Listing 1) and the non-partitioned
    device-memory hash join (Fig. 8 baseline) return exactly the oracle's result."""
    rng = np.random.default_rng(99)
    Rk, Sk = adversarial(rng)[name]
    Rp = rng.integers(0, 1 << 32, len(Rk), dtype=np.uint64).astype(np.uint32)
    Sp = rng.integers(0, 1 << 32, len(Sk), dtype=np.uint64).astype(np.uint32)
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_JOIN_ALGO, algo)
    for bits in (-1, 0, 6):
        check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=bits, mat=True, ctx=ctx)
    ctx.close()


@pytest.mark.parametrize("algo", [1, 2])
@pytest.mark.parametrize("dist,keys", [("fk", "dense"), ("zipf", "sparse"), ("1to1", "k8")])
def test_comparator_algorithms_generated(hj, algo, dist, keys):
    w = W.Workload("t", 1 << 14, 1 << 14, dist, keys=keys, z=1.2, seed=160)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    ctx = hj.Context(0, w.key_bytes, w.key_bytes)
    ctx.set_option(hj.OPT_JOIN_ALGO, algo)
    check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=-1, mat=True, ctx=ctx)
    ctx.close()


@pytest.mark.parametrize("dist,z,rep", [("zipf_build", 0.5, 1), ("zipf_build", 1.0, 1), ("zipf_both", 0.5, 1),
                                        ("zipf_both", 1.0, 1), ("replicas", 0, 2), ("replicas", 0, 4)])
def test_next2_skew_and_replicas_vs_oracle(hj, dist, z, rep):
    """NEXT-2: build-side skew (R co-partitions beyond shared memory -> hash-based block nested
    loops), identical skew (output explosion -> exact growth), replicas."""
    w = W.Workload("t", 1 << 15, 1 << 15, dist, keys="sparse", z=z, rep=rep, seed=170)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=-1, mat=True)


@pytest.mark.slow
@pytest.mark.parametrize("tool", ["memcheck", "racecheck", "synccheck", "initcheck"])
def test_compute_sanitizer_clean(hj, tool):
    import subprocess
    import sys

    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    # racecheck does not model mbarrier hand-offs between warps: it reports hazards on a correct
    # two-warp ping-pong (tools/microbench/mb_mbar_race.cu, profiles/r02_sanitizers.md), so the
    # warp-specialized pass (stages handed over by mbarriers) is excluded from racecheck only
    extra = ["--kernel-name-exclude", "kns=k_pass_ws"] if tool == "racecheck" else []
    out = subprocess.run(["compute-sanitizer", "--tool", tool, *extra, sys.executable,
                          os.path.join(root, "tools", "sanitize_cases.py"), "core"],
                         capture_output=True, text=True, timeout=1800)
    txt = out.stdout + out.stderr
    if "compute-sanitizer is closed" in txt:  # the GPU pool's own policy, not a finding
        pytest.skip("compute-sanitizer is disabled on this GPU pool: " + txt.strip()[:120])
    assert "sanitize cases ok" in txt, txt[-2000:]
    assert ("ERROR SUMMARY: 0 errors" in txt) or ("RACECHECK SUMMARY: 0 hazards" in txt), txt[-2000:]


@pytest.mark.parametrize("timing", [1, 0])
def test_pdl_launch_matches_oracle(hj, timing):
    """HJ_OPT_PDL: the planner, passes and join launched with programmatic dependent launch
    (each waits in-kernel for its predecessor) give the oracle's results, synchronous and queued,
    with and without the per-kernel timing events between the launches."""
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_PDL, 1)
    ctx.set_option(hj.OPT_TIMING, timing)
    w = W.Workload("pdl", 1 << 16, 1 << 18, "zipf", keys="sparse", z=1.0, seed=197)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    cols = [dev(a) for a in (Rk, Rp, Sk, Sp)]
    for _ in range(3):
        res = ctx.join(*cols)
        assert (res.matches, res.checksum) == (m, c)
    for _ in range(4):
        ctx.join_async(*cols, out_mode=hj.OUT_MATERIALIZE)
    for res in ctx.sync():
        assert (res.matches, res.checksum) == (m, c)
    res = ctx.join(*cols, out_mode=hj.OUT_MATERIALIZE)
    assert np.array_equal(oracle.pairs_sorted(to_np(res.r_pay, 4), to_np(res.s_pay, 4)), oracle.pairs_sorted(r, s))
    ctx.close()


def test_graph_replay_matches_oracle(hj):
    """HJ_OPT_GRAPH: the captured launch sequence replays with identical results; a new call
    signature recaptures; materialize overflow falls back to the normal path."""
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_GRAPH, 1)
    for seed in (190, 191):
        w = W.Workload("g", 1 << 14, 1 << 15, "zipf", keys="sparse", z=1.0, seed=seed)
        Rk, Rp, Sk, Sp = W.np_generate(w)
        m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
        cols = [dev(a) for a in (Rk, Rp, Sk, Sp)]
        for _ in range(3):
            res = ctx.join(*cols)
            assert (res.matches, res.checksum) == (m, c)
            assert res.ms_total > 0
        for _ in range(2):
            res = ctx.join(*cols, out_mode=hj.OUT_MATERIALIZE)
            assert res.matches == m
            assert np.array_equal(oracle.pairs_sorted(to_np(res.r_pay, 4), to_np(res.s_pay, 4)), oracle.pairs_sorted(r, s))
    ctx.set_option(hj.OPT_OUT_CAPACITY, 1000)
    Rk = np.repeat(np.arange(50, dtype=np.uint32), 40)
    Sk = np.repeat(np.arange(60, dtype=np.uint32), 30)
    res = check_against_oracle(hj, Rk, np.arange(len(Rk), dtype=np.uint32), Sk, np.arange(len(Sk), dtype=np.uint32),
                               bits=3, mat=True, ctx=ctx)
    assert res.matches == 50 * 40 * 30
    ctx.close()


@pytest.mark.parametrize("variant", [1, 2, 3, 4])
def test_pass_variant_invariance(hj, variant):
    """HJ_OPT_PASS_VARIANT (1024-thread register-prefetch tiles vs 512 threads x twice the tuples,
    per pass) never changes results: skewed, duplicate-heavy and ragged inputs, 4/4 and 8/8."""
    rng = np.random.default_rng(70 + variant)
    for kb in (4, 8):
        ctx = hj.Context(0, kb, kb)
        ctx.set_option(hj.OPT_PASS_VARIANT, variant)
        dt = np.uint32 if kb == 4 else np.uint64
        w = W.Workload("pv", 70001, 90011, "zipf", keys="sparse" if kb == 4 else "k8", z=1.3, seed=420 + variant)
        Rk, Rp, Sk, Sp = W.np_generate(w)
        for bits in (-1, 9, 16):
            check_against_oracle(hj, Rk, Rp, Sk, Sp, bits=bits, mat=bits == 9, ctx=ctx)
        Rk = rng.integers(0, 900, 20000).astype(dt)
        Sk = rng.integers(0, 900, 15000).astype(dt)
        check_against_oracle(hj, Rk, np.arange(len(Rk), dtype=dt), Sk, np.arange(len(Sk), dtype=dt), bits=18,
                             mat=True, ctx=ctx)
        ctx.close()


@pytest.mark.slow
@pytest.mark.timeout(600)
def test_contexts_in_sequence_recycle_memory(hj):
    """Contexts created and closed one after another in one process, alternating the partitioner
    (histogram path <-> bucket chains), at c3's size, joining right after the torch generator
    with no synchronization: each new context's memory is recycled from the closed one's by
    torch's caching allocator (workspace) or cudaMalloc (ctx-owned). Round 1 saw a miscount and a
    hang here: hj_set_stream(NULL) mapped torch's default stream to the ctx's non-blocking
    stream, so the join could read columns the generator was still writing. Every
    join must give the closed form (1:1 permutation: |S| matches, checksum = sum sig(rho(j), j))."""
    w = W.CONFIGS["c3"]
    exp = _closed_form_checksum(w)
    for part in (0, 1, 0, 1):
        cols = W.torch_generate(w, device="cuda")  # no synchronize: the join must be stream-ordered
        ctx = hj.Context(0, w.key_bytes, w.key_bytes)
        ctx.set_option(hj.OPT_PARTITIONER, part)
        for out_mode in (0, w.out_mode):
            r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=out_mode)
            assert (r.matches, r.checksum) == (w.nS, exp), (part, out_mode, r.n_items)
        ctx.close()
        del cols
    torch.cuda.empty_cache()


def _closed_form_checksum(w):
    j = np.arange(w.nS, dtype=np.uint64)
    cdf = W.zipf_cdf(w.nR, w.z) if w.dist == "zipf" else None
    return int(np_sig(W.np_rho_for(w, j, cdf), j).sum(dtype=np.uint64))


@pytest.mark.slow
@pytest.mark.timeout(900)
def test_context_stress_alternating(hj):
    """>= 20 contexts in one process, alternating partitioner (histogram / bucket chains), output
    mode, workspace (torch-owned / ctx-owned) and config (c2 / c3), each joined right after its
    inputs were generated on torch's stream: every result equals the closed form."""
    cfgs = {k: (W.CONFIGS[k], _closed_form_checksum(W.CONFIGS[k])) for k in ("c2", "c3")}
    for i in range(20):
        name = ("c2", "c3")[i % 2]
        w, exp = cfgs[name]
        cols = W.torch_generate(w, device="cuda")
        ctx = hj.Context(0, 4, 4, workspace=(i // 2) % 2 == 0)
        ctx.set_option(hj.OPT_PARTITIONER, (i // 4) % 2)
        mode = (i // 8) % 2
        r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=mode)
        assert (r.matches, r.checksum) == (w.nS, exp), (i, name, mode, r.n_items)
        ctx.close()
        del cols
    torch.cuda.empty_cache()


def test_join_right_after_generation_no_sync(hj):
    """The join is ordered after the producer of its columns on torch's current stream (default
    and a side stream), with no torch.cuda.synchronize() in between."""
    w = W.Workload("ns", 1 << 20, 1 << 22, "fk", keys="sparse", seed=131)
    ref = oracle.hash_join(*W.np_generate(w))
    for use_side in (False, True):
        s = torch.cuda.Stream() if use_side else torch.cuda.current_stream()
        with torch.cuda.stream(s):
            for _ in range(3):
                cols = W.torch_generate(w, device="cuda")
                r = hj.join(*cols)
                assert (r.matches, r.checksum) == ref, use_side


def test_workspace_api(hj):
    """hj_workspace_bytes / hj_set_workspace: hj_join runs inside a caller (torch) buffer that
    starts with garbage (nothing is read before it is written), refuses a too-small one, and the
    binding regrows it when materialized pairs outgrow the capacity (reading S11)."""
    lib = hj.lib()
    w = W.Workload("ws", 1 << 17, 1 << 19, "zipf", keys="sparse", z=1.1, seed=132)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    cols = [dev(a) for a in (Rk, Rp, Sk, Sp)]
    for part in (0, 1):
        ctx = hj.Context(0, 4, 4, workspace=False)
        ctx.set_option(hj.OPT_PARTITIONER, part)
        need = ctx.workspace_bytes(w.nR, w.nS, -1, hj.OUT_MATERIALIZE)
        assert need > 0 and ctx.workspace_bytes(0, w.nS, -1, 0) == 0
        buf = torch.full((need,), 0xA5, dtype=torch.uint8, device="cuda")  # garbage
        assert lib.hj_set_workspace(ctx._h, ctypes.c_void_p(buf.data_ptr() + 8), need) == -1  # unaligned
        small = torch.empty(need // 2, dtype=torch.uint8, device="cuda")
        assert lib.hj_set_workspace(ctx._h, ctypes.c_void_p(small.data_ptr()), small.numel()) == 0
        with pytest.raises(hj.HJError, match="WORKSPACE"):
            ctx.join(*cols, out_mode=hj.OUT_MATERIALIZE)
        assert lib.hj_set_workspace(ctx._h, ctypes.c_void_p(buf.data_ptr()), need) == 0
        for mode in (0, 1, 1):
            res = ctx.join(*cols, out_mode=mode)
            assert (res.matches, res.checksum) == (m, c), (part, mode)
            if mode:
                assert np.array_equal(oracle.pairs_sorted(to_np(res.r_pay, 4), to_np(res.s_pay, 4)),
                                      oracle.pairs_sorted(r, s))
                p0 = res.r_pay.data_ptr()
                assert buf.data_ptr() <= p0 < buf.data_ptr() + need  # the pairs live in the workspace
        assert lib.hj_set_workspace(ctx._h, None, 0) == 0  # back to ctx-owned memory
        res = ctx.join(*cols)
        assert (res.matches, res.checksum) == (m, c)
        ctx.close()
    # the binding's torch workspace regrows on a materialization overflow
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_OUT_CAPACITY, 1000)
    Rk = np.repeat(np.arange(50, dtype=np.uint32), 40)
    Sk = np.repeat(np.arange(60, dtype=np.uint32), 30)
    res = check_against_oracle(hj, Rk, np.arange(len(Rk), dtype=np.uint32), Sk, np.arange(len(Sk), dtype=np.uint32),
                               bits=3, mat=True, ctx=ctx)
    assert res.matches == 50 * 40 * 30
    ctx.close()


def test_join_async_queue_vs_oracle(hj):
    """hj_join_async / hj_sync: more queued calls than HJ_MAX_PENDING (the ring completes the
    oldest), different inputs, sizes, modes and both partitioners on one ctx; every result
    equals the oracle's, in issue order, and the last MATERIALIZE call's pairs are returned."""
    specs = [W.Workload("a%d" % i, n, n if d == "1to1" else 3 * n + i, d, keys=k, z=1.0, seed=140 + i)
             for i, (n, d, k) in enumerate([(1 << 15, "fk", "dense"), (40000, "zipf", "sparse"),
                                            (1 << 16, "1to1", "sparse"), (777, "fk", "sparse")])]
    data = [W.np_generate(w) for w in specs]
    refs = [oracle.hash_join(*a, materialize=True) for a in data]
    cols = [[dev(x) for x in a] for a in data]
    for part, kb in ((0, 4), (1, 4)):
        ctx = hj.Context(0, kb, kb)
        ctx.set_option(hj.OPT_PARTITIONER, part)
        order = [(i % 4, i % 3 == 2) for i in range(2 * hj.MAX_PENDING + 2)] + [(2, True)]
        for i, mat in order:
            ctx.join_async(*cols[i], out_mode=hj.OUT_MATERIALIZE if mat else hj.OUT_COUNT_CHECKSUM)
        out = ctx.sync()
        assert len(out) == len(order)
        for (i, mat), r in zip(order, out):
            assert (r.matches, r.checksum) == refs[i][:2], (part, i, mat)
            assert r.kernels > 0 and r.ms_kernel[4] > 0
        i, mat = order[-1]
        assert mat and np.array_equal(oracle.pairs_sorted(to_np(out[-1].r_pay, 4), to_np(out[-1].s_pay, 4)),
                                      oracle.pairs_sorted(refs[i][2], refs[i][3]))
        # a synchronous call completes pending async calls first (their structs are filled)
        ctx.join_async(*cols[0])
        r = ctx.join(*cols[1])
        assert (r.matches, r.checksum) == refs[1][:2]
        assert [(x.matches, x.checksum) for x in ctx.sync()] == [refs[0][:2]]
        assert ctx.sync() == []
        ctx.close()


def test_join_async_output_overflow_reported_at_sync(hj):
    """A queued MATERIALIZE call whose pairs outgrow the capacity is not re-run (later calls
    reuse the buffers): its completion fails with HJ_ERR_WORKSPACE and the exact count."""
    lib = hj.lib()
    ctx = hj.Context(0, 4, 4, workspace=False)
    ctx.set_option(hj.OPT_OUT_CAPACITY, 1000)
    Rk = np.repeat(np.arange(50, dtype=np.uint32), 40)
    Sk = np.repeat(np.arange(60, dtype=np.uint32), 30)
    cols = [dev(a) for a in (Rk, np.arange(len(Rk), dtype=np.uint32), Sk, np.arange(len(Sk), dtype=np.uint32))]
    res = hj._Result()
    ptrs = [ctypes.c_void_p(c.data_ptr()) for c in cols]
    assert lib.hj_join_async(ctx._h, ptrs[0], ptrs[1], len(Rk), ptrs[2], ptrs[3], len(Sk), 3, 1, ctypes.byref(res)) == 0
    assert lib.hj_sync(ctx._h) == hj.ERR_WORKSPACE
    assert res.matches == 50 * 40 * 30
    assert b"HJ_OPT_OUT_CAPACITY" in lib.hj_last_error(ctx._h)
    assert lib.hj_sync(ctx._h) == 0  # nothing pending any more
    ctx.close()
