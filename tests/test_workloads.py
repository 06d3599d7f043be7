"""CPU tests of the seeded generator (SURVEY.md §8(c.3), §8(c.5) 'Generator' row)."""
import numpy as np
import pytest
import torch

import workloads as W


@pytest.mark.parametrize("k", [1, 2, 5, 12, 16, 20])
def test_perm_pow2_is_bijection(k):
    x = np.arange(1 << k, dtype=np.uint64)
    y = W.np_perm_pow2(12345, k, x)
    assert y.max() < (1 << k)
    assert len(np.unique(y)) == (1 << k)


@pytest.mark.parametrize("n", [1, 3, 1000, 4097, 65535])
def test_perm_n_is_bijection(n):
    y = W.np_perm_n(777, n, np.arange(n, dtype=np.uint64))
    assert sorted(y.tolist()) == list(range(n))


def test_perm_not_identity():
    y = W.np_perm_pow2(5, 16, np.arange(1 << 16, dtype=np.uint64))
    assert (y != np.arange(1 << 16)).mean() > 0.99


@pytest.mark.parametrize("dist", ["fk", "1to1", "zipf"])
@pytest.mark.parametrize("keys", ["dense", "sparse", "k8"])
def test_numpy_and_torch_generators_agree(dist, keys):
    w = W.Workload("t", 1 << 12, 1 << 12, dist, keys=keys, z=1.0, seed=101)
    a = W.np_generate(w)
    b = W.torch_generate(w, device="cpu")
    for x, y in zip(a, b):
        yb = y.numpy().view(np.uint64 if keys == "k8" else np.uint32)
        assert np.array_equal(x.view(yb.dtype), yb)


@pytest.mark.parametrize("nR,nS", [(1000, 3000), (4096, 4096), (1, 7)])
def test_non_pow2_sizes_agree(nR, nS):
    w = W.Workload("t", nR, nS, "fk", seed=103)
    a = W.np_generate(w)
    b = W.torch_generate(w, device="cpu")
    for x, y in zip(a, b):
        assert np.array_equal(x, y.numpy().view(np.uint32))


@pytest.mark.parametrize("keys", ["dense", "sparse", "k8"])
def test_R_keys_unique_and_S_is_foreign_key(keys):
    w = W.Workload("t", 1 << 14, 1 << 15, "fk", keys=keys, seed=104)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    assert len(np.unique(Rk)) == len(Rk)
    assert np.isin(Sk, Rk).all()
    assert np.array_equal(Rp, np.arange(len(Rp)))
    assert np.array_equal(Sp, np.arange(len(Sp)))


def test_dense_keys_are_1_to_n():
    w = W.Workload("t", 1 << 13, 1 << 13, "1to1", seed=105)
    Rk, _, Sk, _ = W.np_generate(w)
    assert sorted(Rk.tolist()) == list(range(1, (1 << 13) + 1))
    assert sorted(Sk.tolist()) == list(range(1, (1 << 13) + 1))  # 1:1 -> S is a permutation of R


def test_s_row_ranges_are_independent():
    w = W.Workload("t", 1 << 12, 1 << 14, "zipf", z=1.5, seed=106)
    _, _, Sk, Sp = W.np_generate(w)
    _, _, Sk2, Sp2 = W.np_generate(w, s_rows=slice(5000, 9000))
    assert np.array_equal(Sk[5000:9000], Sk2) and np.array_equal(Sp[5000:9000], Sp2)


def test_zipf_shape_matches_survey_table():
    # over 2^24 ranks the top-1 key holds 1.2e-4 / 5.8% / 38.3% of S at z = 0.5/1/1.5
    for z, share in [(0.5, 1.2e-4), (1.0, 0.058), (1.5, 0.383)]:
        cdf = W.zipf_cdf(1 << 24, z)
        assert abs(cdf[0] / cdf[-1] - share) / share < 0.05


def test_zipf_empirical_top_share():
    w = W.Workload("t", 1 << 12, 1 << 16, "zipf", z=1.5, seed=107)
    _, _, Sk, _ = W.np_generate(w)
    _, counts = np.unique(Sk, return_counts=True)
    cdf = W.zipf_cdf(1 << 12, 1.5)
    assert abs(counts.max() / len(Sk) - cdf[0] / cdf[-1]) < 0.01


def test_fk_rho_pow2_equals_top_bits():
    # for nR = 2^k the multiply-high map equals rng >> (64 - k)
    j = np.arange(1000, dtype=np.uint64)
    r = W.np_rng(9, W.TAG_U, j)
    assert np.array_equal(W.np_rho("fk", 9, 1 << 10, 1000, j), r >> np.uint64(54))


def test_torch_generator_int32_layout():
    w = W.Workload("t", 1 << 10, 1 << 10, "1to1", seed=108)
    Rk, Rp, Sk, Sp = W.torch_generate(w, device="cpu")
    assert Rk.dtype == torch.int32 and Rk.is_contiguous()


@pytest.mark.parametrize("dist", ["zipf_build", "zipf_both", "replicas"])
@pytest.mark.parametrize("keys", ["dense", "k8"])
def test_next2_generators_agree(dist, keys):
    w = W.Workload("t", 1 << 12, 1 << 13, dist, keys=keys, z=1.0, seed=109, rep=4)
    a = W.np_generate(w)
    b = W.torch_generate(w, device="cpu")
    for x, y in zip(a, b):
        assert np.array_equal(x, y.numpy().view(x.dtype))


def test_next2_shapes():
    # build skew: R has duplicates, S is a permutation of the domain
    w = W.Workload("t", 1 << 14, 1 << 14, "zipf_build", z=1.0, seed=110)
    Rk, _, Sk, _ = W.np_generate(w)
    assert len(np.unique(Sk)) == len(Sk) and np.isin(Rk, Sk).all()
    _, c = np.unique(Rk, return_counts=True)
    assert c.max() > 100  # the top build-side value repeats
    # replicas: every key exactly rep times on each side
    w = W.Workload("t", 1 << 12, 1 << 12, "replicas", rep=4, seed=111)
    Rk, _, Sk, _ = W.np_generate(w)
    assert set(np.unique(Rk, return_counts=True)[1]) == {4}
    assert set(np.unique(Sk, return_counts=True)[1]) == {4}
