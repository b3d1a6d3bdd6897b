"""Shared helpers for the GPU parity tests (CUDA path vs the CPU oracle)."""
import numpy as np
import pytest


def have_gpu() -> bool:
    try:
        import torch
        return torch.cuda.is_available()
    except Exception:
        return False


def require_gpu():
    if not have_gpu():
        pytest.skip("needs a GPU (run under gpurun)")


def rel_l2(got, ref) -> float:
    got = np.asarray(got, dtype=np.float64).ravel()
    ref = np.asarray(ref, dtype=np.float64).ravel()
    den = np.linalg.norm(ref)
    return float(np.linalg.norm(got - ref) / (den if den > 0 else 1.0))


def rel_err_abs(got: float, ref: float, abs_sum: float) -> float:
    """|got - ref| / sum |terms| (signed data)."""
    return abs(float(got) - float(ref)) / max(abs_sum, 1e-300)
