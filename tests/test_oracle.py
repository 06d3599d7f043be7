"""Pins of the CPU oracle against things other than itself.

* published splitmix64 outputs (tests/golden/splitmix64.txt) pin fmix64 -> sig
* a hand-worked join (tests/golden/join_small.txt)
* brute-force nested-loop join (numpy broadcasting) on small adversarial inputs
* numpy sort-merge count sum_k cR(k) * cS(k)
* generator closed forms: FK / 1:1 joins have exactly |S| matches, checksum sum_j sig(rho(j), j),
  and the pairs sorted by s_pay are [(rho(j), j)]
* radix partition vs np.argsort(kind='stable') and np.bincount
"""
import os

import numpy as np
import pytest

import oracle
import workloads as W

GOLDEN = 0x9E3779B97F4A7C15
M64 = (1 << 64) - 1


def sig_py(p, q):
    """Independent python-int evaluation of the pair signature (reading S1), built on the
    generator module's fmix64_int, not on the C oracle."""
    return W.fmix64_int((p ^ (q * GOLDEN)) & M64)


def np_sig(p, q):
    with np.errstate(over="ignore"):
        return W.np_fmix64(p.astype(np.uint64) ^ (q.astype(np.uint64) * np.uint64(GOLDEN)))


def brute_force(Rk, Rp, Sk, Sp):
    eq = Rk[:, None] == Sk[None, :]
    ri, sj = np.nonzero(eq)
    r, s = Rp[ri], Sp[sj]
    chk = 0
    for a, b in zip(r.tolist(), s.tolist()):
        chk = (chk + sig_py(a, b)) & M64
    return len(ri), chk, oracle.pairs_sorted(r, s)


def test_splitmix64_golden(golden_dir):
    for line in open(os.path.join(golden_dir, "splitmix64.txt")):
        if line.startswith("#") or not line.strip():
            continue
        i, hexv = line.split()
        x = (int(i) * GOLDEN) & M64
        assert oracle.fmix64(x) == int(hexv, 16)
        assert W.fmix64_int(x) == int(hexv, 16)


def test_sig_is_pair_sensitive():
    assert oracle.sig(1, 2) != oracle.sig(2, 1)
    assert oracle.sig(3, 4) == sig_py(3, 4)


def test_hand_worked_join(golden_dir):
    R, S, pairs, matches = [], [], [], None
    for line in open(os.path.join(golden_dir, "join_small.txt")):
        f = line.split()
        if not f or f[0].startswith("#"):
            continue
        if f[0] == "R":
            R.append((int(f[1]), int(f[2])))
        elif f[0] == "S":
            S.append((int(f[1]), int(f[2])))
        elif f[0] == "MATCHES":
            matches = int(f[1])
        elif f[0] == "PAIR":
            pairs.append((int(f[1]), int(f[2])))
    Rk = np.array([k for k, _ in R], dtype=np.uint32)
    Rp = np.array([v for _, v in R], dtype=np.uint32)
    Sk = np.array([k for k, _ in S], dtype=np.uint32)
    Sp = np.array([v for _, v in S], dtype=np.uint32)
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    assert m == matches == len(pairs)
    assert [tuple(x) for x in oracle.pairs_sorted(r, s).tolist()] == sorted(pairs)
    exp = 0
    for a, b in pairs:
        exp = (exp + sig_py(a, b)) & M64
    assert c == exp


def _adversarial_cases(rng):
    u32 = np.uint32
    cases = {
        "all_equal": (np.full(300, 5, u32), np.full(200, 5, u32)),
        "disjoint": (np.arange(0, 500, 2, dtype=u32), np.arange(1, 501, 2, dtype=u32)),
        "dups_both": (rng.integers(0, 40, 700).astype(u32), rng.integers(0, 40, 900).astype(u32)),
        "extremes": (np.array([0, 0xFFFFFFFF, 1, 0xFFFFFFFE], u32), np.array([0xFFFFFFFF, 0, 0, 7], u32)),
        "high_bits_only": ((np.arange(64, dtype=u32) << u32(20)) | u32(3), (np.arange(0, 128, dtype=u32) << u32(20)) | u32(3)),
        "empty_R": (np.zeros(0, u32), np.arange(10, dtype=u32)),
        "empty_S": (np.arange(10, dtype=u32), np.zeros(0, u32)),
        "one_row": (np.array([42], u32), np.array([42, 42, 1], u32)),
        "random_ragged": (rng.integers(0, 3000, 4097).astype(u32), rng.integers(0, 3000, 3001).astype(u32)),
    }
    return cases


@pytest.mark.parametrize("name", list(_adversarial_cases(np.random.default_rng(0)).keys()))
def test_oracle_vs_brute_force(name):
    rng = np.random.default_rng(1234)
    Rk, Sk = _adversarial_cases(rng)[name]
    Rp = rng.integers(0, 1 << 32, len(Rk), dtype=np.uint64).astype(np.uint32)
    Sp = rng.integers(0, 1 << 32, len(Sk), dtype=np.uint64).astype(np.uint32)
    m_bf, c_bf, pairs_bf = brute_force(Rk, Rp, Sk, Sp)
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    assert m == m_bf
    assert c == c_bf
    assert np.array_equal(oracle.pairs_sorted(r, s), pairs_bf)
    assert oracle.hash_join(Rk, Rp, Sk, Sp) == (m_bf, c_bf)


def test_oracle_vs_brute_force_8byte():
    rng = np.random.default_rng(5)
    Rk = rng.integers(0, 50, 600, dtype=np.uint64) * np.uint64(0x100000001)
    Sk = rng.integers(0, 50, 500, dtype=np.uint64) * np.uint64(0x100000001)
    Rp = rng.integers(0, 1 << 63, 600, dtype=np.uint64)
    Sp = rng.integers(0, 1 << 63, 500, dtype=np.uint64)
    m_bf, c_bf, pairs_bf = brute_force(Rk, Rp, Sk, Sp)
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    assert (m, c) == (m_bf, c_bf)
    assert np.array_equal(oracle.pairs_sorted(r, s), pairs_bf)


def test_oracle_count_vs_sort_merge():
    rng = np.random.default_rng(7)
    Rk = rng.integers(0, 1 << 16, 200_000).astype(np.uint32)
    Sk = rng.integers(0, 1 << 16, 300_000).astype(np.uint32)
    ur, cr = np.unique(Rk, return_counts=True)
    us, cs = np.unique(Sk, return_counts=True)
    _, ir, is_ = np.intersect1d(ur, us, return_indices=True)
    expected = int((cr[ir].astype(np.int64) * cs[is_].astype(np.int64)).sum())
    m, _ = oracle.hash_join(Rk, np.zeros_like(Rk), Sk, np.zeros_like(Sk))
    assert m == expected


@pytest.mark.parametrize("dist,keys,nR,nS", [("fk", "dense", 1 << 14, 1 << 16), ("1to1", "sparse", 1 << 15, 1 << 15),
                                             ("zipf", "dense", 1 << 12, 1 << 15), ("1to1", "k8", 1 << 13, 1 << 13),
                                             ("fk", "dense", 3000, 5001)])
def test_oracle_closed_form(dist, keys, nR, nS):
    w = W.Workload("t", nR, nS, dist, keys=keys, z=1.5, seed=110)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    rho = W.np_rho_for(w, np.arange(nS, dtype=np.uint64))
    m, c, r, s = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    assert m == nS == W.expected_matches_closed_form(w)
    assert c == int(np_sig(rho, np.arange(nS, dtype=np.uint64)).sum(dtype=np.uint64))
    order = np.argsort(s, kind="stable")
    assert np.array_equal(s[order].astype(np.uint64), np.arange(nS, dtype=np.uint64))
    assert np.array_equal(r[order].astype(np.uint64), rho)


def test_c1_closed_form_full_size():
    w = W.CONFIGS["c1"]
    Rk, Rp, Sk, Sp = W.np_generate(w)
    rho = W.np_rho_for(w, np.arange(w.nS, dtype=np.uint64))
    m, c = oracle.hash_join(Rk, Rp, Sk, Sp)
    assert m == w.nS
    assert c == int(np_sig(rho, np.arange(w.nS, dtype=np.uint64)).sum(dtype=np.uint64))


def test_sliced_mode_sums_to_full():
    w = W.Workload("t", 1 << 13, 1 << 14, "zipf", z=1.0, seed=111)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    full = oracle.hash_join(Rk, Rp, Sk, Sp)
    tot_m, tot_c = 0, 0
    for t in range(8):
        m, c = oracle.hash_join(Rk, Rp, Sk, Sp, slice_bits=3, slice_id=t)
        tot_m += m
        tot_c = (tot_c + c) & M64
        assert 0 < m < full[0]
    assert (tot_m, tot_c) == full


def test_materialize_cap_truncates_but_counts_all():
    Rk = np.array([1, 1, 1], np.uint32)
    Sk = np.array([1, 1], np.uint32)
    m, c, r, s = oracle.hash_join(Rk, np.arange(3, dtype=np.uint32), Sk, np.arange(2, dtype=np.uint32),
                                  materialize=True, cap=4)
    assert m == 6 and len(r) == 4


@pytest.mark.parametrize("bits,shift", [(0, 0), (1, 0), (8, 0), (7, 8), (12, 3)])
def test_radix_partition_vs_stable_argsort(bits, shift):
    rng = np.random.default_rng(bits * 31 + shift)
    keys = rng.integers(0, 1 << 32, 20001, dtype=np.uint64).astype(np.uint32)
    pays = np.arange(len(keys), dtype=np.uint32)
    ok, op, offs = oracle.radix_partition(keys, pays, shift, bits)
    digit = (keys >> np.uint32(shift)) & np.uint32((1 << bits) - 1)
    order = np.argsort(digit, kind="stable")
    assert np.array_equal(ok, keys[order]) and np.array_equal(op, pays[order])
    counts = np.bincount(digit, minlength=1 << bits)
    assert np.array_equal(np.diff(offs.astype(np.int64)), counts)
    assert offs[0] == 0 and offs[-1] == len(keys)


def test_radix_partition_8byte():
    rng = np.random.default_rng(3)
    keys = rng.integers(0, 1 << 63, 5000, dtype=np.uint64)
    pays = rng.integers(0, 1 << 63, 5000, dtype=np.uint64)
    ok, op, offs = oracle.radix_partition(keys, pays, 40, 9)
    digit = (keys >> np.uint64(40)) & np.uint64(511)
    order = np.argsort(digit, kind="stable")
    assert np.array_equal(ok, keys[order]) and np.array_equal(op, pays[order])


def test_copartition_property():
    """Joining co-partitions and summing equals the full join."""
    w = W.Workload("t", 1 << 12, 1 << 13, "fk", keys="sparse", seed=112)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    full = oracle.hash_join(Rk, Rp, Sk, Sp)
    rk, rp, ro = oracle.radix_partition(Rk, Rp, 0, 5)
    sk, sp, so = oracle.radix_partition(Sk, Sp, 0, 5)
    tm, tc = 0, 0
    for p in range(32):
        m, c = oracle.hash_join(rk[ro[p]:ro[p + 1]], rp[ro[p]:ro[p + 1]], sk[so[p]:so[p + 1]], sp[so[p]:so[p + 1]])
        tm += m
        tc = (tc + c) & M64
    assert (tm, tc) == full


@pytest.mark.parametrize("dist,z,rep", [("zipf_build", 1.0, 1), ("zipf_both", 0.75, 1), ("replicas", 0, 2),
                                        ("replicas", 0, 4)])
def test_oracle_next2_vs_sort_merge(dist, z, rep):
    """NEXT-2 workloads (Fig. 17 build-side / identical skew, Fig. 19 replicas): the oracle's count
    equals sum_k cR(k) * cS(k) and the closed form where one exists."""
    w = W.Workload("t", 1 << 13, 1 << 13, dist, z=z, rep=rep, seed=112)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    ur, cr = np.unique(Rk, return_counts=True)
    us, cs = np.unique(Sk, return_counts=True)
    _, ir, is_ = np.intersect1d(ur, us, return_indices=True)
    expected = int((cr[ir].astype(np.int64) * cs[is_].astype(np.int64)).sum())
    m, _ = oracle.hash_join(Rk, Rp, Sk, Sp)
    assert m == expected
    cf = W.expected_matches_closed_form(w)
    if cf is not None:
        assert m == cf
