"""Pins for the oracle's VLC codec, encoder and decoder (-m "not gpu").

Paper pins: Table 3 (App. B), Fig. 2 (:387-399), Fig. 5 (:1001-1050), Fig. 1 (:326-352).
Derived pins: tests/golden/derived_examples.txt (FORMAT.md worked examples).  Invariants: round trip, bit-length
identity, segment layout (R16-R18), error cases (R6, R7, R19).
"""
import numpy as np
import pytest

import oracle as O
from graphs import random_graph, adjacency_lists
from conftest import read_golden


# ---------------------------------------------------------------------------------------------------------------
# VLC
# ---------------------------------------------------------------------------------------------------------------
def test_table3_codewords_exact():
    """All 24 codewords of Table 3 (gamma, zeta2, zeta3)."""
    g = read_golden("table3.txt")
    assert len(g) == 8
    for x, (gam, z2, z3) in g.items():
        x = int(x)
        assert O.vlc_string(1, x) == gam
        assert O.vlc_string(2, x) == z2
        assert O.vlc_string(3, x) == z3


def test_appendix_b_prose_example():
    """App. B :1878-1888 / :2095-2096: 6 = '110'; gamma unary '001'+'10' (leading 1 implicit in the prose, i.e.
    '00110' with it), zeta2 unary '01' + '0110', zeta3 unary '1' + '110'."""
    assert O.vlc_string(1, 6) == "00110"
    assert O.vlc_string(2, 6) == "01" + "0110"
    assert O.vlc_string(3, 6) == "1" + "110"


@pytest.mark.parametrize("k", [1, 2, 3, 4, 5])
def test_vlc_round_trip_and_length(k):
    rng = np.random.default_rng(k)
    xs = [1, 2, 3, 7, 8, 255, 256, (1 << 31) - 1, 1 << 31, (1 << 32) + 1, (1 << 34) - 1]
    xs += [int(v) for v in rng.integers(1, 1 << 34, size=200)]
    bits = "".join(O.vlc_string(k, x) for x in xs)
    b, nb = O.bits_to_bytes(bits)
    pos = 0
    for x in xs:
        s = O.vlc_string(k, x)
        assert len(s) == O.vlc_len(k, x)
        v, pos2 = O.vlc_read(k, b, nb, pos)
        assert v == x and pos2 - pos == len(s)
        pos = pos2
    assert pos == nb


def test_gamma_codes_longer_than_64_bits():
    """gamma(x) for x >= 2^32 is 65+ bits (a hard case for any 64-bit-window decoder)."""
    x = (1 << 33) + 12345
    s = O.vlc_string(1, x)
    assert len(s) == 67
    b, nb = O.bits_to_bytes("1" + s + "1")
    assert O.vlc_read(1, b, nb, 1) == (x, 68)


def test_fig5_vals_and_poss_from_arbitrary_offsets(golden):
    """Fig. 5 round 0: thread i decodes gamma at bit i (e.g. thread 10 reads 20, thread 11 reads 10)."""
    g = golden("fig5.txt")
    bits = g["bits"][0]
    b, nb = O.bits_to_bytes(bits)
    vals = [int(v) for v in g["vals"]]
    poss = [int(v) for v in g["poss0"]]
    for i in range(int(g["K"][0])):
        v, p = O.vlc_read(1, b, nb, i)
        assert (v, p) == (vals[i], poss[i])


# ---------------------------------------------------------------------------------------------------------------
# Alg. 4 parallel decode (Fig. 5, Lemma 5.2)
# ---------------------------------------------------------------------------------------------------------------
def _xs(row):
    return [-1 if t == "x" else int(t) for t in row]


def test_fig5_alg4_trace_exact(golden):
    g = golden("fig5.txt")
    K = int(g["K"][0])
    vals, poss, flags, results, rounds = O.alg4_trace(g["bits"][0], K)
    assert list(vals) == [int(v) for v in g["vals"]]
    assert rounds == 4  # initial state + 3 marking rounds
    for r in range(4):
        assert list(poss[r]) == _xs(g[f"poss{r}"]), r
        assert list(flags[r]) == [int(v) for v in g[f"flags{r}"]], r
    assert list(results) == [int(v) for v in g["results"]]


@pytest.mark.parametrize("k", [1, 3])
def test_alg4_lemma52_round_bound_and_results(k):
    """Lemma 5.2 (:1051-1085): after marking round r the first 2^r valid decodings are marked, so at most
    ceil(log2(#valid)) marking rounds; results equal the serial decode of codes starting in the window."""
    rng = np.random.default_rng(52 + k)
    for trial in range(200):
        xs = [int(v) for v in rng.integers(1, 40, size=40)]
        bits = "".join(O.vlc_string(k, x) for x in xs)
        K = int(rng.choice([8, 16, 32, 64]))
        vals, poss, flags, results, rounds = O.alg4_trace(bits, K, zeta_k=k, max_rounds=32)
        # serial reference: codewords that start inside the first K bits
        serial, pos = [], 0
        for x in xs:
            if pos >= K:
                break
            serial.append(x)
            pos += O.vlc_len(k, x)
        assert list(results) == serial
        nvalid = len(serial)
        marking_rounds = rounds - 1
        assert marking_rounds <= max(0, int(np.ceil(np.log2(nvalid)))) + 1
        # the loop (line 12) stops exactly when every marked thread points past the window
        assert marking_rounds >= int(np.ceil(np.log2(nvalid))) if nvalid > 1 else True


# ---------------------------------------------------------------------------------------------------------------
# Encoder: paper + derived worked examples
# ---------------------------------------------------------------------------------------------------------------
def test_fig2_illustrative_55_bits(golden):
    g = golden("fig2.txt")
    s = O.encode_list(int(g["u"][0]), [int(v) for v in g["list"]], int(g["min_interval_len"][0]), 0, 1,
                      illustrative=True)
    assert s == g["bits"][0]
    assert len(s) == 55  # ":456-457 ... can be denoted with only 55 bits"


def _derived():
    rows, extra = [], {}
    with open(__import__("conftest").GOLDEN + "/derived_examples.txt") as f:
        for line in f:
            line = line.strip()
            if not line or line.startswith("#"):
                continue
            if "|" in line:
                u, lst, ml, sl, k, exp = [t.strip() for t in line.split("|")]
                rows.append((int(u), [int(v) for v in lst.split()], int(ml), int(sl), int(k), exp))
            else:
                key, *rest = line.split()
                extra[key] = rest
    return rows, extra


@pytest.mark.parametrize("row", _derived()[0])
def test_derived_examples(row):
    u, lst, ml, sl, k, exp = row
    s = O.encode_list(u, lst, ml, sl, k)
    if exp.startswith("len="):
        assert len(s) == int(exp[4:])
    else:
        assert s == exp.replace(" ", "")
    # and the record decodes back to the list
    b, nb = O.bits_to_bytes(s)
    got, end = O.decode_vertex(b, nb, 0, u, ml, sl, k)
    assert list(got) == lst and end == nb


def test_fig1_graph_bytes(golden):
    g = golden("fig1.txt")
    _, extra = _derived()
    ro = np.array([int(v) for v in g["row_offsets"]], dtype=np.uint64)
    co = np.array([int(v) for v in g["cols"]], dtype=np.uint32)
    for k, name in [(1, "gamma"), (3, "zeta3")]:
        b, nb, offs = O.encode(ro, co, 4, 0, k)
        assert [int(v) for v in offs] == [int(v) for v in extra[f"fig1_{name}_offsets"]]
        assert b.tobytes().hex() == extra[f"fig1_{name}_bytes"][0]


# ---------------------------------------------------------------------------------------------------------------
# Encoder invariants
# ---------------------------------------------------------------------------------------------------------------
PARAMS = [(ml, sl, k) for k in (1, 2, 3, 4, 5) for ml in (0, 2, 3, 4, 5, 10) for sl in (0, 4, 8, 16, 32, 64, 128)]


@pytest.mark.parametrize("ml,sl,k", PARAMS)
def test_round_trip_random(ml, sl, k):
    for seed, (n, m) in enumerate([(1, 0), (7, 20), (64, 400), (300, 3000)]):
        ro, co = random_graph(n, m, seed=seed * 31 + k) if m else (np.zeros(2, np.uint64), np.zeros(0, np.uint32))
        b, nb, offs = O.encode(ro, co, ml, sl, k)
        assert b.size == (nb + 7) // 8 and int(offs[-1]) == nb
        if nb % 8:
            assert int(b[-1]) & ((1 << (8 - nb % 8)) - 1) == 0  # R1 zero padding
        ro2, co2 = O.decode(b, offs, ml, sl, k, int(ro[-1]))
        assert np.array_equal(ro2, ro) and np.array_equal(co2, co)


def _runs(lst, ml):
    itv, res, i = [], [], 0
    while i < len(lst):
        j = i + 1
        while j < len(lst) and lst[j] == lst[j - 1] + 1:
            j += 1
        if ml and j - i >= ml:
            itv.append((lst[i], j - i))
        else:
            res.extend(lst[i:j])
        i = j
    return itv, res


def _sm(x):
    return 2 * x if x >= 0 else 2 * (-x) + 1


@pytest.mark.parametrize("k", [1, 2, 3, 5])
@pytest.mark.parametrize("ml", [0, 2, 4])
def test_unsegmented_bit_length_identity(k, ml):
    """Record length = sum of the code lengths of R8-R12's fields, counted here field by field."""
    ro, co = random_graph(500, 6000, seed=7 + k)
    b, nb, offs = O.encode(ro, co, ml, 0, k)
    for u, lst in enumerate(adjacency_lists(ro, co)):
        itv, res = _runs(lst, ml)
        L = O.vlc_len(k, len(lst) + 1) + O.vlc_len(k, len(itv) + 1)
        prev_end = None
        for s, l in itv:
            L += O.vlc_len(k, _sm(s - u) + 1 if prev_end is None else s - prev_end)
            L += O.vlc_len(k, l - ml + 1)
            prev_end = s + l - 1
        for i, r in enumerate(res):
            L += O.vlc_len(k, _sm(r - u) + 1 if i == 0 else r - res[i - 1])
        assert int(offs[u + 1] - offs[u]) == L


@pytest.mark.parametrize("k", [1, 3])
@pytest.mark.parametrize("sl", [4, 8, 32])
def test_segment_layout_invariants(k, sl):
    """R16-R18: non-last segments are exactly segBits and each decodes standalone from its start (count + first
    residual anchored at u); the last is <= 2*segBits; a full segment is maximal (one more residual would not fit)."""
    segBits = 8 * sl
    n = 4000
    rng = np.random.default_rng(sl * 10 + k)
    # hubs with long residual lists force many segments
    src = np.concatenate([rng.integers(0, 20, size=20000), rng.integers(0, n, size=8000)])
    dst = rng.integers(0, n, size=src.size)
    from graphs import csr_from_edges
    ro, co = csr_from_edges(n, src, dst)
    b, nb, offs = O.encode(ro, co, 4, sl, k)
    bits = O.bytes_to_bits(b, nb)
    bb, _ = O.bits_to_bytes(bits)
    nsegs_seen = 0
    for u, lst in enumerate(adjacency_lists(ro, co)):
        itv, res = _runs(lst, 4)
        p = int(offs[u])
        v, p = O.vlc_read(k, bb, nb, p)
        assert v == len(itv) + 1
        for _ in range(2 * len(itv)):
            _, p = O.vlc_read(k, bb, nb, p)
        v, p = O.vlc_read(k, bb, nb, p)
        segNum = v - 1
        base, got = p, []
        for j in range(segNum):
            q = base + j * segBits
            cnt, q = O.vlc_read(k, bb, nb, q)
            cnt -= 1
            assert cnt >= 1
            seg = []
            for t in range(cnt):
                v, q = O.vlc_read(k, bb, nb, q)
                if t == 0:
                    z = v - 1
                    seg.append(u + (-(z >> 1) if z & 1 else z >> 1))
                else:
                    seg.append(seg[-1] + v)
            if j + 1 < segNum:
                assert q - (base + j * segBits) <= segBits
                assert set(bits[q: base + (j + 1) * segBits]) <= {"0"}  # blank padding
                # maximality: adding the next residual would overflow segBits
                nxt = res[len(got) + cnt]
                extra = O.vlc_len(k, nxt - seg[-1]) + O.vlc_len(k, cnt + 2) - O.vlc_len(k, cnt + 1)
                assert (q - (base + j * segBits)) + extra > segBits
            else:
                assert q - (base + j * segBits) <= 2 * segBits
                assert q == int(offs[u + 1])
            got.extend(seg)
            nsegs_seen += 1
        assert got == res
        if segNum == 0:
            assert p == int(offs[u + 1])
    assert nsegs_seen > 50


def test_input_validation():
    ro = np.array([0, 2, 2], dtype=np.uint64)
    with pytest.raises(O.OracleError) as e:
        O.encode(ro, np.array([1, 1], dtype=np.uint32), 4, 0, 3)  # duplicate (R6)
    assert e.value.code == -2
    with pytest.raises(O.OracleError) as e:
        O.encode(ro, np.array([1, 0], dtype=np.uint32), 4, 0, 3)  # unsorted (R6)
    assert e.value.code == -2
    with pytest.raises(O.OracleError) as e:
        O.encode(ro, np.array([0, 5], dtype=np.uint32), 4, 0, 3)  # id >= n
    assert e.value.code == -3
    with pytest.raises(O.OracleError) as e:
        O.encode(ro, np.array([0, 1], dtype=np.uint32), 1, 0, 3)  # minLen 1 (R7)
    assert e.value.code == -1
    # R19: 1-byte segments cannot hold a far residual (gamma: header 3 bits + a long code)
    n = 1000
    ro = np.array([0] + [3] * n, dtype=np.uint64)
    co = np.array([100, 500, 900], dtype=np.uint32)
    with pytest.raises(O.OracleError) as e:
        O.encode(ro, co, 4, 1, 1)
    assert e.value.code == -4


@pytest.mark.parametrize("threads", [1, 4, 8])
def test_encode_par_byte_identical(threads):
    """The per-vertex-parallel oracle encoder (chunks concatenated at the prefix sum of their bit lengths, R2) is
    byte-identical to the serial orc_encode, across chunk boundaries (n > 65536) and every parameter family."""
    import synth
    from graphs import random_graph
    cases = [random_graph(1, 0, seed=1), random_graph(70_000, 400_000, seed=threads),
             synth.CONFIGS["web_s"].make(), synth.CONFIGS["social_s"].make()]
    for ro, co in cases:
        for ml, sl, k in [(4, 32, 3), (0, 0, 1), (2, 8, 5), (4, 0, 2)]:
            b, nb, offs = O.encode(ro, co, ml, sl, k)
            pb, pnb, poffs = O.encode_par(ro, co, ml, sl, k, threads)
            assert nb == pnb and np.array_equal(offs, poffs) and np.array_equal(b, pb), (ml, sl, k)
    for ro, co, code in [([0, 2, 2], [1, 1], -2), ([0, 1, 1], [5], -3)]:  # duplicate id (R6), id >= n
        with pytest.raises(O.OracleError) as e:
            O.encode_par(np.array(ro, np.uint64), np.array(co, np.uint32), 4, 32, 3)
        assert e.value.code == code
