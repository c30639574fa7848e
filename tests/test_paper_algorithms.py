"""The paper's worked examples (tests/golden/) pin the step-by-step replays of Algorithms 1 and 2
(oracle/paper_algorithms.py), and the replays agree with the plain-definition oracle."""
import os
import re

import numpy as np
import pytest

import oracle
from oracle import paper_algorithms as pa

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")
RNG = np.random.default_rng(7)


def _lines(name):
    with open(os.path.join(GOLDEN, name)) as fh:
        return [ln.strip() for ln in fh if ln.strip() and not ln.startswith("#")]


def _kv(name):
    d = {}
    for ln in _lines(name):
        parts = ln.split()
        d.setdefault(parts[0], []).append(parts[1:])
    return d


# ---------------------------------------------------------------- Fig. 1 / Algorithm 1
def test_fig1a_direct_elements_golden():
    g = _kv("fig1_column_reuse.txt")
    row = np.arange(64, dtype=np.float32)  # value == element index
    win, loads, shuffles = pa.fig1a_direct_k5(row)
    assert (loads, shuffles) == (5, 0)
    for t, *elems in g["direct"]:
        tid = int(t[1:])
        assert [int(v) for v in win[tid]] == [int(e) for e in elems]


@pytest.mark.parametrize("base", [0, 32, 96, 7])
def test_alg1_third_element_every_lane(base):
    row = np.arange(200, dtype=np.float32) * np.float32(1.25) - 3
    it = [[row[base + t], 0, 0, 0, row[base + t + 4]] for t in range(32)]
    out = pa.alg1_retrieve_third_element(it)
    for t in range(32):
        assert np.float32(out[t][2]).view(np.uint32) == row[base + t + 2].view(np.uint32)


def test_alg1_random_bits_exact():
    row = RNG.standard_normal(64).astype(np.float32)
    row[5] = np.float32("-0.0")
    row[9] = np.float32(1e-42)  # denormal survives the 64-bit pack/shift/unpack
    it = [[row[t], 0, 0, 0, row[t + 4]] for t in range(32)]
    out = pa.alg1_retrieve_third_element(it)
    assert all(np.float32(out[t][2]).view(np.uint32) == row[t + 2].view(np.uint32) for t in range(32))


def test_fig1c_windows_and_counts_golden():
    g = _kv("fig1_column_reuse.txt")
    assert [int(v) for v in g["fig1c_offsets"][0]] == [0, 1, 2, 3, 4]
    steps = [int(v) for v in g["fig1c_steps"][0]]
    # steps 1 and 2 are the loads at offsets 0 and 4; step 3 (Algorithm 1) is offset 2
    assert steps[0] == 1 and steps[4] == 2 and steps[2] == 3 and sorted(steps) == [1, 2, 3, 4, 5]
    row = RNG.standard_normal(100).astype(np.float32)
    for base in (0, 32, 40):
        win, loads, shuffles = pa.fig1c_column_reuse_k5(row, base)
        assert loads == int(g["fig1c_loads_per_thread"][0][0])
        assert shuffles == int(g["fig1c_shuffles_per_thread"][0][0])
        for t in range(32):
            assert np.array_equal(np.array(win[t], np.float32), row[base + t:base + t + 5])
    # Fig. 1b: offsets 0, 2, 4 -- Algorithm 1 alone provides the middle element
    assert [int(v) for v in g["fig1b_offsets"][0]] == [0, 2, 4]


# ---------------------------------------------------------------- Fig. 2 / Algorithm 2
_EQ = re.compile(r"out(\d+) = (.*)")
_TERM = re.compile(r"rowi(\d+) · rowf(\d+)")


def _fig2():
    eqs, flow, direct, reuse = {}, [], None, None
    cur = None
    for ln in _lines("fig2_row_reuse.txt"):
        if ln.startswith("direct_row_loads"):
            direct = int(ln.split()[1])
            continue
        if ln.startswith("reuse_row_loads"):
            reuse = int(ln.split()[1])
            continue
        if ln.startswith("load rowi"):
            cur = int(re.match(r"load rowi(\d+)", ln).group(1))
            ln = ln.split(":", 1)[1].strip()
            flow.append(("load", cur))
        m = _EQ.match(ln)
        o = int(m.group(1))
        terms = [(int(a), int(b)) for a, b in _TERM.findall(m.group(2))]
        if cur is None:
            eqs[o] = terms
        else:
            assert len(terms) == 1 and terms[0][0] == cur
            flow.append(("update", cur, o, terms[0][1]))
    return eqs, flow, direct, reuse


def test_fig2_equations_match_oracle():
    eqs, _, direct, _ = _fig2()
    FH, IH, IW = 3, 5, 3 + 4
    img = synth_int((IH, IW))
    f = synth_int((FH, FH))
    out, _, _ = oracle.conv2d_single(img, f)
    assert out.shape == (3, IW - FH + 1)
    for o, terms in eqs.items():
        exp = np.zeros(IW - FH + 1)
        for (ri, rf) in terms:
            exp += np.array([np.dot(img[ri, x:x + FH].astype(np.float64), f[rf].astype(np.float64))
                             for x in range(IW - FH + 1)])
        assert np.array_equal(out[o].astype(np.float64), exp)
    assert direct == sum(len(t) for t in eqs.values()) == pa.direct_row_loads(IH, FH)


def synth_int(shape):
    return RNG.integers(-8, 9, shape).astype(np.float32)


def test_fig2_flow_is_algorithm2_trace():
    """The re-ordered flow printed at P:303-311 is exactly Algorithm 2's update sequence (with the
    DESIGN.md R8 fix of case 3), and it loads 5 rows instead of 9."""
    _, flow, direct, reuse = _fig2()
    exp = [(r, o, k) for (tag, *rest) in flow if tag == "update" for (r, o, k) in [tuple(rest)]]
    img = synth_int((5, 6))
    f = synth_int((3, 3))
    trace = []
    Out, loads = pa.alg2_row_reuse(img, f, trace)
    assert trace == exp
    assert loads == reuse == 5 and direct == 9
    trace_g = []
    Out_g, _ = pa.alg2_general(img, f, trace_g)
    assert trace_g == exp and np.array_equal(Out, Out_g)
    out, _, _ = oracle.conv2d_single(img, f)
    assert np.array_equal(Out.astype(np.float32), out)


def test_algorithm2_equals_direct_definition():
    for FH in range(1, 16):
        for IH in sorted({max(FH, 2 * FH - 2), 2 * FH + 3, 40}):
            img = RNG.standard_normal((IH, FH + 5)).astype(np.float32)
            f = RNG.standard_normal((FH, FH)).astype(np.float32)
            _, bound, out64 = oracle.conv2d_single(img, f, want_f64=True)
            Out, loads = pa.alg2_row_reuse(img, f)
            assert loads == IH
            assert (np.abs(Out - out64) <= 1e-12 * bound).all()


def test_general_rule_short_images():
    """For IH < 2FH-2 the printed cases overlap; the general rule (R9) still equals the definition."""
    for FH in range(3, 16):
        for IH in range(FH, 2 * FH - 2):
            img = RNG.standard_normal((IH, FH + 3)).astype(np.float32)
            f = RNG.standard_normal((FH, FH)).astype(np.float32)
            _, bound, out64 = oracle.conv2d_single(img, f, want_f64=True)
            Out, loads = pa.alg2_general(img, f)
            assert loads == IH and (np.abs(Out - out64) <= 1e-12 * bound).all()
            with pytest.raises(ValueError):
                pa.alg2_row_reuse(img, f)
