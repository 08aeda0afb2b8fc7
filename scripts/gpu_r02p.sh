for c in 0 1 2 3 4; do timeout 60 ./scripts/probes/tma_store_probe $c; done
