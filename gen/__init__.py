"""Seeded synthetic inputs; see gen/synth.py. Holds none of the method's arithmetic."""
from .synth import (BASE_SEED, FILTER_DISTS, IMAGE_DISTS, TAG_FILTER, TAG_INPUT, fill_np,
                    fill_torch, hash_np, make_filter, splitmix64_np)

__all__ = ["BASE_SEED", "FILTER_DISTS", "IMAGE_DISTS", "TAG_FILTER", "TAG_INPUT", "fill_np",
           "fill_torch", "hash_np", "make_filter", "splitmix64_np"]
