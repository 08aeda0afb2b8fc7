"""G4: the device generator (tds_generate, csrc/gen.cu) draws exactly the
host generator's systems (inputs.py, SURVEY §8(d) "implemented twice ...
checked bit-equal"): both dtypes, shard offsets (first_system), padded
strides, margins; the BASELINE configs' batches compared element by element."""
import numpy as np
import pytest

from paper_conf_ipps_davidsonzo11_b200 import inputs

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def tds():
    import torch
    assert torch.cuda.is_available()
    import paper_conf_ipps_davidsonzo11_b200 as m
    m._lib.load()
    return m


@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("n,m,seed,first,mu", [(1, 3, 1, 0, 1.0), (2, 5, 7, 0, 1.0), (1000, 7, 3, 0, 1.0),
                                                (1000, 4, 3, 3, 1.0), (4097, 3, 2 ** 63 + 5, 11, 0.01),
                                                (65536, 9, 102, 256, 0.5)])
def test_generate_bit_identical(tds, dtype, n, m, seed, first, mu):
    import torch
    name = "float32" if dtype == np.float32 else "float64"
    fam = "dd" if mu == 1.0 else "weak"
    kw = {"mu": mu} if fam == "dd" else {"param": mu}
    ref = inputs.generate(n, m, dtype, seed=seed, family=fam, first_system=first, **kw)
    got = tds.generate(n, m, name, seed=seed, first_system=first, mu=mu)
    torch.cuda.synchronize()
    for r, g in zip(ref, got):
        g = g.cpu().numpy()
        assert g.dtype == dtype
        assert np.array_equal(r.view(np.uint8), g.view(np.uint8))  # bit-identical (incl. signed zeros)


def test_generate_padded_stride_untouched(tds):
    import torch
    n, m, stride = 1000, 3, 1012
    out = tuple(torch.full((m, stride), 7.0, dtype=torch.float32, device="cuda") for _ in range(4))
    tds.generate(n, m, "float32", seed=9, batch_stride=stride, out=out)
    torch.cuda.synchronize()
    ref = inputs.generate(n, m, np.float32, seed=9)
    for r, g in zip(ref, out):
        g = g.cpu().numpy()
        assert np.array_equal(g[:, :n], r) and np.all(g[:, n:] == 7.0)


@pytest.mark.parametrize("cfg,dtype", [(3, np.float32), (3, np.float64), (4, np.float32)])
def test_generate_config_batches(tds, cfg, dtype):
    """The whole batch bench.py times (config seeds)."""
    import torch
    n, m = {3: (1 << 20, 16), 4: (16384, 4096)}[cfg]
    seed = inputs.config_seed(cfg, dtype)
    got = tds.generate(n, m, "float32" if dtype == np.float32 else "float64", seed=seed)
    torch.cuda.synchronize()
    ref = inputs.generate(n, m, dtype, seed=seed)
    for r, g in zip(ref, got):
        assert np.array_equal(r, g.cpu().numpy())


def test_generate_shards_equal_whole(tds):
    """Rank r of G draws systems [r m/G, (r+1) m/G) of the unsharded batch."""
    import torch
    n, m, G = 4096, 16, 4
    whole = [t.cpu() for t in tds.generate(n, m, "float32", seed=5)]
    for r in range(G):
        part = tds.generate(n, m // G, "float32", seed=5, first_system=r * (m // G))
        torch.cuda.synchronize()
        for w, p in zip(whole, part):
            assert torch.equal(w[r * (m // G):(r + 1) * (m // G)], p.cpu())


def test_generate_argument_errors(tds):
    import ctypes
    lib = tds._lib.load()
    assert lib.tds_generate(0, 0, 1, 0, 1, 0, 1.0, 16, 16, 16, 16, None) == 1      # n < 1
    assert lib.tds_generate(0, 10, 1, 5, 1, 0, 1.0, 16, 16, 16, 16, None) == 1     # stride < n
    assert lib.tds_generate(2, 10, 1, 0, 1, 0, 1.0, 16, 16, 16, 16, None) == 1     # dtype
    assert lib.tds_generate(0, 10, 1, 0, 1, 0, 1.0, None, 16, 16, 16, None) == 1   # NULL
    assert lib.tds_generate(1, 10, 1, 0, 1, 0, 1.0, 20, 16, 16, 16, None) == 1     # misaligned fp64
    assert ctypes is not None
