"""Profile-guided sharing ratios (DESIGN.md R-solver-11): the oracle against
closed forms, the library against the oracle (CPU only)."""
import numpy as np
import pytest

from oracle import guided_ref as G

FR = [1.0, 0.75, 0.5, 0.375, 0.25, 0.1875, 0.125, 0.0625]


def linear(T):
    return [T / f for f in FR]


def saturating(T, fs):
    return [T * max(1.0, fs / f) for f in FR]


def test_identical_profiles_equal_weights():
    w, pred, S, fr = G.guided_weights(FR, [linear(2.0)] * 4)
    assert w == [16] * 4 and all(abs(x - 0.25) < 1e-9 for x in fr) and abs(S - 4.0) < 1e-9


def test_linear_profiles_any_length():
    """s = 1/f for every request: equal fractions whatever the absolute times."""
    w, pred, S, fr = G.guided_weights(FR, [linear(0.5), linear(3.0), linear(7.0)])
    assert w == [16, 16, 16] and abs(S - 3.0) < 1e-9


def test_saturating_next_to_linear():
    """A kernel at full speed from f = 1/4 up (s = 1/(4f) below) next to a
    linear one (s = 1/f): 1/S + 1/(4S) = 1 -> S = 5/4, f = (4/5, 1/5),
    weights 16 : 4, both predicted 5/4."""
    w, pred, S, fr = G.guided_weights(FR, [linear(1.0), saturating(1.0, 0.25)])
    assert abs(S - 1.25) < 1e-9 and abs(fr[0] - 0.8) < 1e-9 and abs(fr[1] - 0.2) < 1e-9
    assert w == [16, 4]
    assert abs(pred[0] - 1.25) < 1e-9 and abs(pred[1] - 1.25) < 1e-9


def test_everything_fits():
    """Kernels saturated at 1/4 each, two of them: no slowdown, S = 1."""
    w, pred, S, fr = G.guided_weights(FR, [saturating(1.0, 0.25)] * 2)
    assert S == 1.0 and pred == [1.0, 1.0] and w == [16, 16]


def test_non_monotone_profile_is_smoothed():
    """A measured blip (faster at a smaller share) never predicts a larger
    share to be slower."""
    f, s = G.slowdown_curve(FR, [1.0, 1.3, 1.1, 1.5, 2.0, 2.5, 3.5, 7.0])
    assert all(s[j] >= s[j + 1] for j in range(len(s) - 1))


def test_library_matches_oracle():
    from paper_conf_cgo_margiolaso16_b200 import abi
    r = np.random.Generator(np.random.PCG64(5))
    for trial in range(40):
        k = int(r.integers(1, 9))
        ms = []
        for _ in range(k):
            T = float(r.uniform(0.2, 8.0))
            beta = float(r.uniform(0.0, 1.1))
            noise = r.uniform(0.95, 1.05, len(FR))
            row = [T * (1.0 / f) ** beta * n for f, n in zip(FR, noise)]
            row[0] = T
            ms.append(row)
        w_c, p_c = abi.accel_guided_weights(FR, ms)
        w_o, p_o, S, fr = G.guided_weights(FR, ms)
        assert w_c == w_o, (trial, w_c, w_o)
        assert np.allclose(p_c, p_o, rtol=1e-9, atol=1e-12)


def test_library_rejects_bad_profiles():
    from paper_conf_cgo_margiolaso16_b200 import abi
    with pytest.raises(abi.AccelError):
        abi.accel_guided_weights([0.5, 1.0], [[1.0, 2.0]])
    with pytest.raises(abi.AccelError):
        abi.accel_guided_weights(FR, [[0.0] * len(FR)])
